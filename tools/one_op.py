"""Run one op a few times (for ncu --set full captures).  usage: one_op.py OP M N [algo]"""
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import synth  # noqa: E402
import paper_conf_cgo_steuwerrd17_b200 as lift  # noqa: E402

op, m, n = sys.argv[1], int(sys.argv[2]), int(sys.argv[3])
extra = sys.argv[4] if len(sys.argv) > 4 else "auto"
dev = torch.device("cuda:0")
if op == "dot":
    x = synth.torch_uniform(0, 0, m, device=dev)
    y = synth.torch_uniform(1, 0, m, device=dev)
    f = lambda: lift.lift_dot(x, y)  # noqa: E731
else:
    A = synth.torch_matrix_rows(2, n, 0, m, device=dev)
    x = synth.torch_uniform(0, 0, n, device=dev)
    if op == "gemv":
        f = lambda: lift.lift_gemv(A, x)  # noqa: E731
    elif op == "gesummv":
        B = synth.torch_matrix_rows(3, n, 0, m, device=dev)
        f = lambda: lift.lift_gesummv(1.5, A, 1.2, B, x)  # noqa: E731
    elif op == "atax":
        f = lambda: lift.lift_atax(A, x, algo=extra)  # noqa: E731
for _ in range(3):
    f()
torch.cuda.synchronize()
