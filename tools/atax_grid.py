"""Fused-ATAX grid-size probe (tuning aid, not part of the library).

The library launches k_atax_fused with one block per SM (cooperative).  The
explicit block count of the NVLink entry point (lift_atax_reduce with a
simulated one-rank exchange, plain launch) lets this probe time other grid
sizes: fewer blocks mean fewer partial rows to sum and, at 128 blocks for
8192 rows, no ragged last round of rows.  Every call reads its own copy of A
(copies > 2x L2); eager back-to-back calls timed with CUDA events.
usage: python tools/atax_grid.py
"""
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import synth  # noqa: E402
import paper_conf_cgo_steuwerrd17_b200 as lift  # noqa: E402
from paper_conf_cgo_steuwerrd17_b200 import nvlink  # noqa: E402

dev = torch.device("cuda:0")
sms = torch.cuda.get_device_properties(dev).multi_processor_count


def time_calls(calls, reps=3):
    for c in calls[:2]:
        c()
    torch.cuda.synchronize()
    best = 1e30
    for _ in range(reps):
        s, e = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        s.record()
        for c in calls:
            c()
        e.record()
        e.synchronize()
        best = min(best, s.elapsed_time(e) * 1e3 / len(calls))
    return best


for m, n, sets in ((8192, 8192, 3), (4096, 4096, 8), (16384, 8192, 2)):
    As = [synth.torch_matrix_rows(2 + 10 * k, n, 0, m, device=dev) for k in range(sets)]
    x = synth.torch_uniform(0, 0, n, device=dev)
    y = torch.empty(n, device=dev)
    ref = lift.lift_atax(As[0], x, algo="fused").clone()
    (ex,) = nvlink.ExchangeArea.simulated(nvlink.EXCH_REDUCE, n, 1, dev)
    ws = torch.zeros(lift.lib().lift_atax_workspace_bytes(m, n), dtype=torch.uint8, device=dev)
    calls = [(lambda A=A: lift.lift_atax(A, x, out=y, algo="fused")) for A in (As * 30)[:30]]
    t = time_calls(calls)
    by = 4 * m * n + 8 * n
    print(f"atax {m}x{n} library (cooperative, {sms} blocks): {t:8.2f} us  {by / t / 1e3:8.1f} GB/s", flush=True)
    for blocks in (sms, 144, 136, 128, 120, 112, 96, 74):
        got = nvlink.lift_atax_reduce(As[0], x, ex, dst=0, blocks=blocks, workspace=ws)
        # a different block count sums in a different order: compare at the scale of y
        # (tools/atax_blocks_check.py checks each against fp64 with the north_star tolerance)
        assert (got - ref).abs().max() <= 1e-5 * ref.abs().max(), blocks
        calls = [(lambda A=A, b=blocks: nvlink.lift_atax_reduce(A, x, ex, dst=0, out=y, blocks=b, workspace=ws))
                 for A in (As * 30)[:30]]
        t = time_calls(calls)
        print(f"atax {m}x{n} exch1 blocks {blocks:4d} rows/block {m / blocks:6.2f}: {t:8.2f} us  "
              f"{by / t / 1e3:8.1f} GB/s", flush=True)
