"""Cost of the in-kernel collective epilogue (tuning aid): each op at the
per-rank share of an 8-GPU run, plain kernel vs the same kernel with its
collective fused in (world 1: one exchange area, so only the epilogue —
publish, acquire, copy-out, acknowledge — differs).  24 calls per CUDA graph
(the exchange epoch lives on the device, so fused calls capture), operands
rotated past L2, best of 3 replays.
usage: python tools/fused_overhead.py"""
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, os.environ.get("LIFT_ROOT") or os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import synth  # noqa: E402
import paper_conf_cgo_steuwerrd17_b200 as lift  # noqa: E402
from paper_conf_cgo_steuwerrd17_b200 import nvlink  # noqa: E402
from sweep import graph_time  # noqa: E402

dev = torch.device("cuda:0")
L2 = torch.cuda.get_device_properties(dev).L2_cache_size


def sets_of(make, nbytes):
    return [make(k) for k in range(max(2, -(-3 * L2 // nbytes)))]


# GESUMMV / GEMV 8192^2 at 8 ranks: 1024 rows each; ATAX 8192^2: 1024 rows; dot 2^31 / 8 and 2^20 / 8
for name, m, n in (("gemv", 1024, 8192), ("gemv", 512, 4096), ("atax", 1024, 8192)):
    As = sets_of(lambda k: synth.torch_matrix_rows(2 + 10 * k, n, 0, m, device=dev), 4 * m * n)
    x = synth.torch_uniform(0, 0, n, device=dev)
    if name == "gemv":
        y = torch.empty(m, device=dev)
        ex = nvlink.ExchangeArea.simulated(nvlink.EXCH_GATHER, m, 1, dev)[0]
        ws = torch.zeros(256, dtype=torch.uint8, device=dev)
        plain = [(lambda A=A: lift.lift_gemv(A, x, out=y)) for A in (As * 24)[:24]]
        fused = [(lambda A=A: nvlink.lift_gemv_allgather(A, x, 0, m, ex, out=y, workspace=ws)) for A in (As * 24)[:24]]
    else:
        y = torch.empty(n, device=dev)
        ex = nvlink.ExchangeArea.simulated(nvlink.EXCH_REDUCE, n, 1, dev)[0]
        ws = torch.zeros(nvlink.workspace_bytes("atax", m, n), dtype=torch.uint8, device=dev)
        plain = [(lambda A=A: lift.lift_atax(A, x, out=y, algo="fused")) for A in (As * 24)[:24]]
        fused = [(lambda A=A: nvlink.lift_atax_reduce(A, x, ex, dst=-1, out=y, workspace=ws)) for A in (As * 24)[:24]]
    tp, tf = graph_time(plain), graph_time(fused)
    print(f"{name} {m}x{n}: plain {tp:7.2f} us  fused (world 1) {tf:7.2f} us  epilogue {tf - tp:+6.2f} us", flush=True)
    del As
for n in (1 << 28, 1 << 17):
    xs = sets_of(lambda k: synth.torch_uniform(50 + k, 0, n, device=dev), 4 * n)
    r = torch.empty((), device=dev)
    ex = nvlink.ExchangeArea.simulated(nvlink.EXCH_DOT, 0, 1, dev)[0]
    ws = torch.zeros(nvlink.workspace_bytes("dot", 0, n), dtype=torch.uint8, device=dev)
    plain = [(lambda v=v: lift.lift_dot(v, v, out=r)) for v in (xs * 24)[:24]]
    fused = [(lambda v=v: nvlink.lift_dot_allreduce(v, v, ex, out=r, workspace=ws)) for v in (xs * 24)[:24]]
    tp, tf = graph_time(plain), graph_time(fused)
    print(f"dot {n}: plain {tp:7.2f} us  fused (world 1) {tf:7.2f} us  epilogue {tf - tp:+6.2f} us", flush=True)
    del xs
