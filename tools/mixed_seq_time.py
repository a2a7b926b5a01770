"""Time ATAX in the bench step's context (tuning aid): a CUDA graph of
sequences [GESUMMV 8192^2, ATAX 8192^2, GEMV 4096^2] over rotating operands
(> 2x L2 in total), against the same graph without the ATAX — the difference
is the ATAX's cost inside a mixed stream of kernels (launch gaps and
programmatic-dependent-launch overlap included), not alone.
usage: python tools/mixed_seq_time.py"""
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, os.environ.get("LIFT_ROOT") or os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import synth  # noqa: E402
import paper_conf_cgo_steuwerrd17_b200 as lift  # noqa: E402
from sweep import graph_time  # noqa: E402

dev = torch.device("cuda:0")
sets = 2
G = [(synth.torch_matrix_rows(2 + k, 8192, 0, 8192, device=dev), synth.torch_matrix_rows(3 + k, 8192, 0, 8192, device=dev))
     for k in range(sets)]
T = [synth.torch_matrix_rows(5 + k, 8192, 0, 8192, device=dev) for k in range(sets)]
S = [synth.torch_matrix_rows(7 + k, 4096, 0, 4096, device=dev) for k in range(4)]
x8, x4 = synth.torch_uniform(0, 0, 8192, device=dev), synth.torch_uniform(1, 0, 4096, device=dev)
y8, z8, y4 = torch.empty(8192, device=dev), torch.empty(8192, device=dev), torch.empty(4096, device=dev)


def seq(k, with_atax):
    c = [lambda A=G[k % sets][0], B=G[k % sets][1]: lift.lift_gesummv(1.5, A, 1.2, B, x8, out=y8)]
    if with_atax:
        c.append(lambda A=T[k % sets]: lift.lift_atax(A, x8, out=z8))
    c.append(lambda A=S[k % 4]: lift.lift_gemv(A, x4, out=y4))
    return c


for rep in range(3):
    n = 8
    with_ = graph_time([f for k in range(n) for f in seq(k, True)]) * 3
    without = graph_time([f for k in range(n) for f in seq(k, False)]) * 2
    print(f"sequence with ATAX {with_:8.2f} us   without {without:8.2f} us   ATAX in context {with_ - without:7.2f} us",
          flush=True)
