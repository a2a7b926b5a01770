"""ATAX fused vs two-pass timing (graph of back-to-back calls), tuning aid."""
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import synth  # noqa: E402
sys.path.insert(0, os.path.dirname(os.path.abspath(__file__)))
import paper_conf_cgo_steuwerrd17_b200 as lift  # noqa: E402
from sweep import graph_time  # noqa: E402

dev = torch.device("cuda:0")
for m, n, sets in ((4096, 4096, 4), (8192, 8192, 1), (16384, 8192, 1), (2000, 16384, 2)):
    As = [synth.torch_matrix_rows(2 + 10 * k, n, 0, m, device=dev) for k in range(sets)]
    x = synth.torch_uniform(0, 0, n, device=dev)
    y = torch.empty(n, device=dev)
    for algo in ("fused", "twopass"):
        calls = [(lambda A=A: lift.lift_atax(A, x, out=y, algo=algo)) for A in (As * 12)[:12]]
        t = graph_time(calls)
        mult = 4 if algo == "fused" else 8
        print(f"atax {algo:8s} {m}x{n}: {t:9.2f} us  {mult * m * n / t / 1e3:8.1f} GB/s (alg bytes {mult}mn)", flush=True)
    del As
