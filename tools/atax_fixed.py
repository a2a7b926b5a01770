"""Fixed vs per-row cost of the fused ATAX kernel (tuning aid).

usage: python tools/atax_fixed.py [n]   (each call reads its own copy of A: HBM, not L2)
"""
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
sys.path.insert(0, os.path.dirname(os.path.abspath(__file__)))
import synth  # noqa: E402
import paper_conf_cgo_steuwerrd17_b200 as lift  # noqa: E402
from sweep import graph_time  # noqa: E402

dev = torch.device("cuda:0")
n = int(sys.argv[1]) if len(sys.argv) > 1 else 8192
l2 = torch.cuda.get_device_properties(dev).L2_cache_size
pool = synth.torch_uniform(2, 0, 3 << 28, device=dev)  # 3 GiB
x = synth.torch_uniform(0, 0, n, device=dev)
for m in (148, 296, 592, 1184, 2368, 4096, 4736, 8192, 16384):
    per = m * n
    copies = min(pool.numel() // per, int(-(-2 * l2 // (4 * per))) + 1)
    As = [pool[k * per:(k + 1) * per].view(m, n) for k in range(copies)]
    reps = max(12, copies)
    y = torch.empty(n, device=dev)
    for algo in ("fused", "twopass"):
        t = graph_time([(lambda A=A: lift.lift_atax(A, x, out=y, algo=algo)) for A in (As * reps)[:reps]])
        print(f"atax {algo:8s} m={m:6d} n={n}: {t:8.2f} us  {4 * per / t / 1e3:7.1f} GB/s(4mn)", flush=True)
    yg = torch.empty(m, device=dev)
    t = graph_time([(lambda A=A: lift.lift_gemv(A, x, out=yg)) for A in (As * reps)[:reps]])
    print(f"gemv          m={m:6d} n={n}: {t:8.2f} us  {4 * per / t / 1e3:7.1f} GB/s", flush=True)
