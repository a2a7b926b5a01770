"""Fused-ATAX ring depth x row assignment sweep (lift_atax_fused_tuned).
(Round 1 also swept an L2 bulk-prefetch distance, since removed from the
library: profiles/r01r_atax_tune.txt.)

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
    grid = [(nst, cyc) for cyc in (0, 1) for nst in (0, 2, 3, 4, 5, 6)]
    if quick:
        grid = [(nst, cyc) for cyc in (0, 1) for nst in (0, 3, 4)]
    for nst, cyc in grid:
        try:
            got = lift.lift_atax_fused_tuned(As[0], x, nst=nst, cyclic=cyc)
        except lift.LiftError as e:
            print(f"atax {m}x{n} cyc {cyc} nst {nst}: {e}", flush=True)
            continue
        if cyc == 1:  # the automatic assignment: bitwise the library call for every ring depth
            assert torch.equal(got, ref), nst
        else:
            assert torch.allclose(got, ref, rtol=1e-4, atol=1e-3), nst
        calls = [(lambda A=A: lift.lift_atax_fused_tuned(A, x, out=y, nst=nst, cyclic=cyc)) for A in (As * 12)[:12]]
        t = graph_time(calls)
        print(f"atax {m}x{n} cyc {cyc} nst {nst}: {t:8.2f} us  {4 * m * n / t / 1e3:8.1f} GB/s", flush=True)
    del As
