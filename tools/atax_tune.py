"""Fused-ATAX ring depth x L2 prefetch distance sweep (lift_atax_fused_tuned).

Each timed call reads a different copy of A (copies totalling > 2x L2), so
every call streams A from HBM; time per call from a CUDA graph of 12 calls.
usage: python tools/atax_tune.py [--quick]
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
quick = "--quick" in sys.argv
shapes = ((8192, 8192, 2), (4096, 4096, 5)) if not quick else ((8192, 8192, 2),)
for m, n, sets in shapes:
    As = [synth.torch_matrix_rows(2 + 10 * k, n, 0, m, device=dev) for k in range(sets)]
    x = synth.torch_uniform(0, 0, n, device=dev)
    y = torch.empty(n, device=dev)
    ref = lift.lift_atax(As[0], x, algo="fused").clone()
    grid = [(nst, l2a, cyc) for cyc in (0, 1) for nst in (0, 2, 3, 4, 5, 6) for l2a in (0, 1, 2, 4)]
    if quick:
        grid = [(nst, 0, cyc) for cyc in (0, 1) for nst in (0, 3, 4)]
    for nst, l2a, cyc in grid:
        try:
            got = lift.lift_atax_fused_tuned(As[0], x, nst=nst, l2_ahead=l2a, cyclic=cyc)
        except lift.LiftError as e:
            print(f"atax {m}x{n} cyc {cyc} nst {nst} l2a {l2a}: {e}", flush=True)
            continue
        if cyc == 0:
            assert torch.equal(got, ref), (nst, l2a)
        else:
            assert torch.allclose(got, ref, rtol=1e-4, atol=1e-3), (nst, l2a)
        calls = [(lambda A=A: lift.lift_atax_fused_tuned(A, x, out=y, nst=nst, l2_ahead=l2a, cyclic=cyc))
                 for A in (As * 12)[:12]]
        t = graph_time(calls)
        print(f"atax {m}x{n} cyc {cyc} nst {nst} l2a {l2a}: {t:8.2f} us  {4 * m * n / t / 1e3:8.1f} GB/s",
              flush=True)
    del As
