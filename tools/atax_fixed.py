"""Fixed vs per-row cost of the fused ATAX kernel (tuning aid)."""
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
sys.path.insert(0, os.path.dirname(os.path.abspath(__file__)))
import synth  # noqa: E402
import paper_conf_cgo_steuwerrd17_b200 as lift  # noqa: E402
from sweep import graph_time  # noqa: E402

dev = torch.device("cuda:0")
n = 8192
for m in (148, 296, 592, 1184, 2368, 4736, 8192, 16384):
    A = synth.torch_matrix_rows(2, n, 0, m, device=dev)
    x = synth.torch_uniform(0, 0, n, device=dev)
    y = torch.empty(n, device=dev)
    for algo in ("fused", "twopass"):
        t = graph_time([(lambda: lift.lift_atax(A, x, out=y, algo=algo))] * 10)
        print(f"{algo:8s} m={m:6d} n={n}: {t:8.2f} us", flush=True)
    xg = torch.empty(m, device=dev)
    t = graph_time([(lambda: lift.lift_gemv(A, x, out=xg))] * 10)
    print(f"gemv     m={m:6d} n={n}: {t:8.2f} us", flush=True)
    xd = synth.torch_uniform(0, 0, m * n, device=dev)
    t = graph_time([(lambda: lift.lift_dot(xd, xd))] * 10)
    print(f"dot      n={m*n:9d}: {t:8.2f} us", flush=True)
    del A, xd
