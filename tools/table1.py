"""The paper's Table-1 sizes (and configs[0]'s dot) one at a time, for ncu.

    python tools/table1.py            time every size (CUDA graph, like bench.py)
    python tools/table1.py NAME       run NAME's call 4 times on distinct operands
                                      (under ncu: tools/gpu_round.sh)
"""
import os
import sys

import torch

# LIFT_ROOT: the package root to time (tools/ab_tree.sh points it at an older tree)
ROOT = os.environ.get("LIFT_ROOT") or os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
sys.path.insert(0, os.path.join(ROOT, "tools"))
import bench  # noqa: E402
import synth  # noqa: E402
import paper_conf_cgo_steuwerrd17_b200 as lift  # noqa: E402

dev = torch.device("cuda:0")
l2 = torch.cuda.get_device_properties(dev).L2_cache_size
pool = synth.torch_uniform(synth.SEED_A, 0, (3 << 30) // 4 * 1, device=dev)  # 3 GiB of operands
dx = synth.torch_uniform(synth.SEED_X, 0, 1 << 29, device=dev)  # 2 GiB: two copies of the 2^28 dots
dy = synth.torch_uniform(synth.SEED_Y, 0, 1 << 29, device=dev)
sets = bench.table1_calls(lift, pool, dx, dy, dev, l2)
want = sys.argv[1] if len(sys.argv) > 1 else None
for name, op, shp, algo, calls in sets:
    if want is not None:
        if name != want:
            continue
        for j in range(4):  # (cycles when there are fewer copies; ncu flushes L2 before each launch)
            calls[j % len(calls)]()
        torch.cuda.synchronize()
        break
    if os.environ.get("TABLE1_ONLY") and name not in os.environ["TABLE1_ONLY"].split(","):
        continue
    from sweep import graph_time  # noqa: E402

    reps = max(20, len(calls))
    t = graph_time([calls[j % len(calls)] for j in range(reps)])
    by = bench.alg_bytes(op, shp, algo)
    print(f"{name:24s} {t:9.2f} us  {by / t / 1e3:8.1f} GB/s", flush=True)
