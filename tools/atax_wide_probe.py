"""Single-pass ATAX for wide rows (cluster kernel) against the two-pass
algorithm: time per call (12 calls per CUDA graph on rotated copies of A,
> 2x L2; median of 5 replays).  usage: python tools/atax_wide_probe.py"""
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, os.getcwd())  # run from a package root (this tree or a patched copy)
import synth  # noqa: E402
import paper_conf_cgo_steuwerrd17_b200 as lift  # noqa: E402
from sweep import graph_time  # noqa: E402

dev = torch.device("cuda:0")
L2 = torch.cuda.get_device_properties(dev).L2_cache_size
print(f"# {torch.cuda.get_device_name(dev)}  L2 {L2 >> 20} MiB", flush=True)
SHAPES = ((2048, 32768), (8192, 32768), (4096, 65536), (8192, 49152), (8192, 24576), (16384, 16416), (8192, 20000),
          (1024, 131072))
if os.environ.get("WIDE_QUICK"):
    SHAPES = ((8192, 32768), (4096, 65536))
if os.environ.get("WIDE_SHAPES"):  # e.g. "8192x16384,16384x16384"
    SHAPES = tuple(tuple(int(v) for v in s.split("x")) for s in os.environ["WIDE_SHAPES"].split(","))
for m, n in SHAPES:
    sets = max(2, -(-2 * L2 // (4 * m * n)))
    As = [synth.torch_matrix_rows(2 + 10 * k, n, 0, m, device=dev) for k in range(sets)]
    x = synth.torch_uniform(0, 0, n, device=dev)
    y = torch.empty(n, device=dev)
    a = lift.lift_atax(As[0], x, algo="fused")
    b = lift.lift_atax(As[0], x, algo="twopass")
    rel = ((a - b).abs().max() / b.abs().max()).item()
    res = {}
    for algo in ("fused", "twopass"):
        res[algo] = graph_time([(lambda A=A: lift.lift_atax(A, x, out=y, algo=algo)) for A in (As * 12)[:12]])
    gb = 4 * m * n / 1e3
    print(f"atax {m}x{n}: fused {res['fused']:8.2f} us ({gb / res['fused']:7.1f} GB/s of 4mn)   "
          f"two-pass {res['twopass']:8.2f} us   speedup {res['twopass'] / res['fused']:.2f}x   "
          f"max rel diff {rel:.1e}", flush=True)
    del As
