"""Collectives fused into the kernels (include/lift_nvlink.h, NEXT-2), run as
`world` simulated ranks on ONE GPU: every rank's exchange area is a separate
HBM allocation, all ranks share one peer table, and each rank's kernel is
launched on its own stream so the ranks run concurrently — the same kernels
and the same flag / epoch / parity protocol a multi-GPU run uses over NVLink
(only the transport differs: same-device stores instead of NVLink stores).
"""
import numpy as np
import pytest
import torch

import oracle
import synth
import paper_conf_cgo_steuwerrd17_b200 as lift
from paper_conf_cgo_steuwerrd17_b200 import nvlink
from paper_conf_cgo_steuwerrd17_b200.shard import partition_rows

pytestmark = [pytest.mark.gpu, pytest.mark.timeout(300)]


def run_ranks(world, fn):
    """fn(rank) launches rank's work on the current stream; all ranks concurrently.
    Everything fn touches must be allocated beforehand: an allocation inside the
    launch loop may synchronise the device while rank 0 waits for rank 1."""
    streams = [torch.cuda.Stream() for _ in range(world)]
    outs = [None] * world
    torch.cuda.synchronize()
    for r in range(world):
        with torch.cuda.stream(streams[r]):
            outs[r] = fn(r)
    torch.cuda.synchronize()
    return outs


def prealloc(world, op, m, n, out_shape, device):
    ws = [torch.zeros(nvlink.workspace_bytes(op, m, n), dtype=torch.uint8, device=device) for _ in range(world)]
    outs = [torch.empty(out_shape, dtype=torch.float32, device=device) for _ in range(world)]
    torch.cuda.synchronize()
    return ws, outs


@pytest.mark.parametrize("world", [1, 2, 3, 4, 8])
def test_dot_allreduce_sim(cuda_device, world):
    n = (1 << 20) + 13
    x = synth.torch_uniform(synth.SEED_X, 0, n, device=cuda_device)
    y = synth.torch_uniform(synth.SEED_Y, 0, n, device=cuda_device)
    exs = nvlink.ExchangeArea.simulated(nvlink.EXCH_DOT, 0, world, cuda_device)
    parts = [partition_rows(n, world, r) for r in range(world)]
    ref, mag = oracle.dot(x.cpu().numpy(), y.cpu().numpy())
    ws, res = prealloc(world, "dot", 0, n, (), cuda_device)
    for it in range(3):  # successive epochs exercise the parity double buffer
        outs = run_ranks(world, lambda r: nvlink.lift_dot_allreduce(x[parts[r][0]:parts[r][1]],
                                                                    y[parts[r][0]:parts[r][1]], exs[r],
                                                                    out=res[r], workspace=ws[r]))
        vals = [o.item() for o in outs]
        assert all(np.float32(v).view(np.uint32) == np.float32(vals[0]).view(np.uint32) for v in vals)
        ok, margin = oracle.within_tol([vals[0]], [ref], [mag])
        assert ok, margin
        # exactly the rank-order sum of the per-rank dots
        per = [lift.lift_dot(x[a:b], y[a:b]).item() for a, b in parts]
        s = np.float32(0)
        for v in per:
            s = np.float32(s + np.float32(v))
        assert np.float32(vals[0]) == s


@pytest.mark.parametrize("world", [2, 3, 4, 8])
@pytest.mark.parametrize("op", ["gemv", "gesummv"])
def test_gemv_allgather_sim(cuda_device, world, op):
    m, n = 1000, 4096
    A = synth.torch_matrix_rows(synth.SEED_A, n, 0, m, device=cuda_device)
    B = synth.torch_matrix_rows(synth.SEED_B, n, 0, m, device=cuda_device)
    x = synth.torch_uniform(synth.SEED_X, 0, n, device=cuda_device)
    full = lift.lift_gemv(A, x) if op == "gemv" else lift.lift_gesummv(1.5, A, 1.2, B, x)
    exs = nvlink.ExchangeArea.simulated(nvlink.EXCH_GATHER, m, world, cuda_device)
    parts = [partition_rows(m, world, r) for r in range(world)]
    ws, res = prealloc(world, op, m, n, (m,), cuda_device)
    for it in range(3):
        outs = run_ranks(world, lambda r: nvlink.lift_gemv_allgather(
            A[parts[r][0]:parts[r][1]], x, parts[r][0], m, exs[r], out=res[r], workspace=ws[r],
            B=None if op == "gemv" else B[parts[r][0]:parts[r][1]], alpha=1.5, beta=1.2))
        for r in range(world):
            assert torch.equal(outs[r], full), (r, it)  # bitwise: canonical row order


@pytest.mark.parametrize("world", [1, 2, 4])
@pytest.mark.parametrize("dst", [-1, 0, 1])
def test_atax_reduce_sim(cuda_device, world, dst):
    if dst >= world:
        pytest.skip("dst outside the group")
    m, n = 3000, 4096
    A = synth.torch_matrix_rows(synth.SEED_A, n, 0, m, device=cuda_device)
    x = synth.torch_uniform(synth.SEED_X, 0, n, device=cuda_device)
    ref, mag = oracle.atax(A.cpu().numpy(), x.cpu().numpy())
    exs = nvlink.ExchangeArea.simulated(nvlink.EXCH_REDUCE, n, world, cuda_device)
    parts = [partition_rows(m, world, r) for r in range(world)]
    blocks = 148 // world  # every rank's blocks co-resident on the one GPU
    ws, res = prealloc(world, "atax", m, n, (n,), cuda_device)
    for it in range(2):
        outs = run_ranks(world, lambda r: nvlink.lift_atax_reduce(A[parts[r][0]:parts[r][1]], x, exs[r], dst=dst,
                                                                  blocks=blocks, out=res[r], workspace=ws[r]))
        dsts = range(world) if dst < 0 else [dst]
        for r in dsts:
            ok, margin = oracle.within_tol(outs[r].cpu().numpy(), ref, mag)
            assert ok, (r, margin)
            assert torch.equal(outs[r], outs[dsts[0]])


def test_atax_reduce_rank_with_no_rows(cuda_device):
    world, n = 3, 512
    A = synth.torch_matrix_rows(synth.SEED_A, n, 0, 2, device=cuda_device)  # 2 rows over 3 ranks
    x = synth.torch_uniform(synth.SEED_X, 0, n, device=cuda_device)
    ref, mag = oracle.atax(A.cpu().numpy(), x.cpu().numpy())
    exs = nvlink.ExchangeArea.simulated(nvlink.EXCH_REDUCE, n, world, cuda_device)
    parts = [partition_rows(2, world, r) for r in range(world)]
    assert parts[0][1] - parts[0][0] == 0
    ws, res = prealloc(world, "atax", 2, n, (n,), cuda_device)
    outs = run_ranks(world, lambda r: nvlink.lift_atax_reduce(A[parts[r][0]:parts[r][1]], x, exs[r], dst=-1,
                                                              blocks=8, out=res[r], workspace=ws[r]))
    for r in range(world):
        ok, margin = oracle.within_tol(outs[r].cpu().numpy(), ref, mag)
        assert ok, margin


def _launch_sequence(world, calls, delay_rank=None, delay_cycles=0):
    """calls[k](r) launches rank r's k-th call on the current stream.  Every rank
    issues all its calls back to back with NO host synchronisation between them;
    `delay_rank`'s stream sleeps before each of its calls, so the other ranks run
    ahead of it as far as the protocol lets them."""
    streams = [torch.cuda.Stream() for _ in range(world)]
    torch.cuda.synchronize()
    for k in range(len(calls)):
        for r in range(world):
            with torch.cuda.stream(streams[r]):
                if r == delay_rank:
                    torch.cuda._sleep(delay_cycles)
                calls[k](r)
    torch.cuda.synchronize()


@pytest.mark.parametrize("world", [2, 3])
def test_atax_reduce_dst_back_to_back_no_sync(cuda_device, world):
    """Reduce-to-one-rank calls back to back, the destination delayed before
    each: the senders never wait for the destination's data, so without the
    consumed-epoch acknowledgement they would store call k + 2's partials into
    the parity buffer the destination is still summing for call k (the race of
    round 1).  Every call's result must match the oracle for ITS x."""
    K, dst = 5, 0
    m, n = 1024, 2048
    A = synth.torch_matrix_rows(synth.SEED_A, n, 0, m, device=cuda_device)
    xs = [synth.torch_uniform(100 + k, 0, n, device=cuda_device) for k in range(K)]
    exs = nvlink.ExchangeArea.simulated(nvlink.EXCH_REDUCE, n, world, cuda_device)
    parts = [partition_rows(m, world, r) for r in range(world)]
    ws = [torch.zeros(nvlink.workspace_bytes("atax", m, n), dtype=torch.uint8, device=cuda_device)
          for _ in range(world)]
    outs = [[torch.full((n,), float("nan"), device=cuda_device) for _ in range(world)] for _ in range(K)]
    blocks = 148 // (world + 1)
    calls = [lambda r, k=k: nvlink.lift_atax_reduce(A[parts[r][0]:parts[r][1]], xs[k], exs[r], dst=dst,
                                                    blocks=blocks, out=outs[k][r], workspace=ws[r])
             for k in range(K)]
    _launch_sequence(world, calls, delay_rank=dst, delay_cycles=400_000)  # ~0.2 ms per call
    An = A.cpu().numpy()
    for k in range(K):
        ref, mag = oracle.atax(An, xs[k].cpu().numpy())
        ok, margin = oracle.within_tol(outs[k][dst].cpu().numpy(), ref, mag)
        assert ok, (k, margin)


@pytest.mark.parametrize("world", [2, 3])
def test_mixed_collectives_back_to_back_no_sync(cuda_device, world):
    """All-reduce, reduce-to-rank-1 and reduce-to-rank-0 ATAX calls interleaved on
    one exchange area, back to back, a different rank delayed each time: the
    device-resident epoch and the acknowledgements keep every call's data apart."""
    m, n = 600, 1024
    A = synth.torch_matrix_rows(synth.SEED_A, n, 0, m, device=cuda_device)
    modes = [-1, 1, 0, 1, -1, 0, 0]
    K = len(modes)
    xs = [synth.torch_uniform(200 + k, 0, n, device=cuda_device) for k in range(K)]
    exs = nvlink.ExchangeArea.simulated(nvlink.EXCH_REDUCE, n, world, cuda_device)
    parts = [partition_rows(m, world, r) for r in range(world)]
    ws = [torch.zeros(nvlink.workspace_bytes("atax", m, n), dtype=torch.uint8, device=cuda_device)
          for _ in range(world)]
    outs = [[torch.full((n,), float("nan"), device=cuda_device) for _ in range(world)] for _ in range(K)]
    blocks = 148 // (world + 1)
    calls = [lambda r, k=k: nvlink.lift_atax_reduce(A[parts[r][0]:parts[r][1]], xs[k], exs[r], dst=modes[k],
                                                    blocks=blocks, out=outs[k][r], workspace=ws[r])
             for k in range(K)]
    for delayed in range(world):
        _launch_sequence(world, calls, delay_rank=delayed, delay_cycles=300_000)
        An = A.cpu().numpy()
        for k in range(K):
            ref, mag = oracle.atax(An, xs[k].cpu().numpy())
            for r in (range(world) if modes[k] < 0 else [modes[k]]):
                ok, margin = oracle.within_tol(outs[k][r].cpu().numpy(), ref, mag)
                assert ok, (delayed, k, r, margin)
