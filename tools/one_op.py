"""Run one op a few times (for ncu --set full captures).  usage: one_op.py OP M N [algo]
OP: dot | partial_dot | dot_listing1 (M = n) | gemv | gesummv | atax [fused|twopass] | sgemv_t"""
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import synth  # noqa: E402
import paper_conf_cgo_steuwerrd17_b200 as lift  # noqa: E402

op, m, n = sys.argv[1], int(sys.argv[2]), int(sys.argv[3])
extra = sys.argv[4] if len(sys.argv) > 4 else "auto"
dev = torch.device("cuda:0")
if op in ("dot", "partial_dot", "dot_listing1"):
    x = synth.torch_uniform(0, 0, m, device=dev)
    y = synth.torch_uniform(1, 0, m, device=dev)
    f = {"dot": lambda: lift.lift_dot(x, y), "partial_dot": lambda: lift.lift_partial_dot(x, y),
         "dot_listing1": lambda: lift.lift_dot_listing1(x, y)}[op]
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
    elif op == "sgemv_t":  # y = A^T x (the transposed SGEMV, NEXT-4)
        xt = synth.torch_uniform(1, 0, m, device=dev)
        f = lambda: lift.lift_sgemv(1.0, A, xt, 0.0, trans=True)  # noqa: E731
for _ in range(3):
    f()
torch.cuda.synchronize()
