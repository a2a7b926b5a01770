"""Check the fused ATAX at explicit block counts against an fp64 reference with the
north_star tolerance |y - y_ref| <= 1e-5 * mag + 1e-6 (mag = |A|^T (|A| |x|)).
usage: python tools/atax_blocks_check.py"""
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import synth  # noqa: E402
import paper_conf_cgo_steuwerrd17_b200 as lift  # noqa: E402
from paper_conf_cgo_steuwerrd17_b200 import nvlink  # noqa: E402

dev = torch.device("cuda:0")
for m, n in ((16384, 8192), (8192, 8192), (4096, 4096)):
    A = synth.torch_matrix_rows(2, n, 0, m, device=dev)
    x = synth.torch_uniform(0, 0, n, device=dev)
    A64, x64 = A.double(), x.double()
    yref = A64.t() @ (A64 @ x64)
    mag = A64.abs().t() @ (A64.abs() @ x64.abs())
    tol = 1e-5 * mag + 1e-6
    lib_y = lift.lift_atax(A, x, algo="fused")
    print(f"{m}x{n} library margin {((lib_y.double() - yref).abs() / tol).max().item():.3e}", flush=True)
    (ex,) = nvlink.ExchangeArea.simulated(nvlink.EXCH_REDUCE, n, 1, dev)
    for blocks in (148, 136, 128, 120, 64):
        ws = torch.zeros(lift.lib().lift_atax_workspace_bytes(m, n), dtype=torch.uint8, device=dev)
        got = nvlink.lift_atax_reduce(A, x, ex, dst=0, blocks=blocks, workspace=ws)
        torch.cuda.synchronize()
        marg = ((got.double() - yref).abs() / tol).max().item()
        d = (got - lib_y).abs()
        print(f"{m}x{n} blocks {blocks}: margin {marg:.3e}  max|got-lib| {d.max().item():.3e} at {d.argmax().item()}"
              f"  |y| there {lib_y[d.argmax()].item():.3e}", flush=True)
