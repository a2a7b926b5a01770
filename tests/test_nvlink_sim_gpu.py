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
    torch.cuda._sleep(1)  # load torch's sleep kernel now: a lazy module load waits for an idle device
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


@pytest.mark.parametrize("seed", [1, 2, 3])
def test_exchange_random_sequences_no_sync(cuda_device, seed):
    """Random sequences of fused calls on simulated ranks, every rank issuing its
    calls back to back with no host synchronisation, a random rank's stream
    delayed by a random amount before each call: ATAX reductions with random
    destinations (-1 = all) on one exchange area and dot all-reduces on another,
    interleaved.  Every call's result must be that call's own (different x per
    call), so no run-ahead or parity mix-up goes unnoticed."""
    rng = np.random.default_rng(seed)
    world = int(rng.integers(2, 5))
    m, n = 300, 512
    A = synth.torch_matrix_rows(synth.SEED_A, n, 0, m, device=cuda_device)
    K = 10
    xs = [synth.torch_uniform(300 + 17 * seed + k, 0, n, device=cuda_device) for k in range(K)]
    nd = 4096 + int(rng.integers(0, 100))
    dvs = [synth.torch_uniform(500 + 17 * seed + k, 0, nd, device=cuda_device) for k in range(K)]
    ex_a = nvlink.ExchangeArea.simulated(nvlink.EXCH_REDUCE, n, world, cuda_device)
    ex_d = nvlink.ExchangeArea.simulated(nvlink.EXCH_DOT, 0, world, cuda_device)
    parts = [partition_rows(m, world, r) for r in range(world)]
    dparts = [partition_rows(nd, world, r) for r in range(world)]
    ws_a = [torch.zeros(nvlink.workspace_bytes("atax", m, n), dtype=torch.uint8, device=cuda_device)
            for _ in range(world)]
    ws_d = [torch.zeros(nvlink.workspace_bytes("dot", 0, nd), dtype=torch.uint8, device=cuda_device)
            for _ in range(world)]
    kinds = rng.integers(0, 2, K)  # 0: ATAX reduce, 1: dot all-reduce
    dsts = rng.integers(-1, world, K)
    delays = [(int(rng.integers(0, world)), int(rng.integers(0, 400_000))) for _ in range(K)]
    outs = [[torch.full((n,) if kinds[k] == 0 else (), float("nan"), device=cuda_device) for _ in range(world)]
            for k in range(K)]
    blocks = 148 // (world + 1)
    streams = [torch.cuda.Stream() for _ in range(world)]
    torch.cuda._sleep(1)  # load torch's sleep kernel now: a lazy module load waits for an idle device,
    torch.cuda.synchronize()  # which ranks spinning on each other's flags never leave
    for k in range(K):
        for r in range(world):
            with torch.cuda.stream(streams[r]):
                if r == delays[k][0]:
                    torch.cuda._sleep(delays[k][1])
                if kinds[k] == 0:
                    nvlink.lift_atax_reduce(A[parts[r][0]:parts[r][1]], xs[k], ex_a[r], dst=int(dsts[k]),
                                            blocks=blocks, out=outs[k][r], workspace=ws_a[r])
                else:
                    a, b = dparts[r]
                    nvlink.lift_dot_allreduce(dvs[k][a:b], dvs[k][a:b], ex_d[r], out=outs[k][r], workspace=ws_d[r])
    torch.cuda.synchronize()
    An = A.cpu().numpy()
    for k in range(K):
        if kinds[k] == 0:
            ref, mag = oracle.atax(An, xs[k].cpu().numpy())
            for r in (range(world) if dsts[k] < 0 else [int(dsts[k])]):
                ok, margin = oracle.within_tol(outs[k][r].cpu().numpy(), ref, mag)
                assert ok, (seed, k, r, margin)
        else:
            v = dvs[k].cpu().numpy()
            ref, mag = oracle.dot(v, v)
            vals = [outs[k][r].item() for r in range(world)]
            assert all(np.float32(a).view(np.uint32) == np.float32(vals[0]).view(np.uint32) for a in vals), (k, vals)
            ok, margin = oracle.within_tol([vals[0]], [ref], [mag])
            assert ok, (seed, k, margin)


@pytest.mark.parametrize("op", ["gemv", "gesummv", "dot"])
def test_rank_with_nothing_to_compute(cuda_device, op):
    """More ranks than rows (elements): a rank with an empty shard still launches
    its kernel and takes part in the exchange, and every rank gets the result."""
    world = 4
    if op == "dot":
        nd = 3
        x = synth.torch_uniform(synth.SEED_X, 0, 64, device=cuda_device)[:nd]
        exs = nvlink.ExchangeArea.simulated(nvlink.EXCH_DOT, 0, world, cuda_device)
        parts = [partition_rows(nd, world, r) for r in range(world)]
        assert any(b - a == 0 for a, b in parts)
        ws, res = prealloc(world, "dot", 0, 64, (), cuda_device)
        outs = run_ranks(world, lambda r: nvlink.lift_dot_allreduce(x[parts[r][0]:parts[r][1]],
                                                                    x[parts[r][0]:parts[r][1]], exs[r],
                                                                    out=res[r], workspace=ws[r]))
        ref, mag = oracle.dot(x.cpu().numpy(), x.cpu().numpy())
        for o in outs:
            ok, margin = oracle.within_tol([o.item()], [ref], [mag])
            assert ok, margin
        return
    m, n = 3, 512
    A = synth.torch_matrix_rows(synth.SEED_A, n, 0, m, device=cuda_device)
    B = synth.torch_matrix_rows(synth.SEED_B, n, 0, m, device=cuda_device)
    x = synth.torch_uniform(synth.SEED_X, 0, n, device=cuda_device)
    full = lift.lift_gemv(A, x) if op == "gemv" else lift.lift_gesummv(1.5, A, 1.2, B, x)
    exs = nvlink.ExchangeArea.simulated(nvlink.EXCH_GATHER, m, world, cuda_device)
    parts = [partition_rows(m, world, r) for r in range(world)]
    assert any(b - a == 0 for a, b in parts)
    ws, res = prealloc(world, op, m, n, (m,), cuda_device)
    for it in range(2):
        outs = run_ranks(world, lambda r: nvlink.lift_gemv_allgather(
            A[parts[r][0]:parts[r][1]], x, parts[r][0], m, exs[r], out=res[r], workspace=ws[r],
            B=None if op == "gemv" else B[parts[r][0]:parts[r][1]], alpha=1.5, beta=1.2))
        for r in range(world):
            assert torch.equal(outs[r], full), (r, it)


def test_fused_binding_rejects_wrong_extents(cuda_device):
    """The fused entry points' outputs, inputs and exchange areas are checked
    against the call's shape before any launch (the kernels store by the call's
    m / n into buffers whose extent they cannot see)."""
    m, n = 64, 256
    A = synth.torch_matrix_rows(synth.SEED_A, n, 0, m, device=cuda_device)
    x = synth.torch_uniform(synth.SEED_X, 0, n, device=cuda_device)
    ex_dot = nvlink.ExchangeArea.simulated(nvlink.EXCH_DOT, 0, 1, cuda_device)[0]
    ex_g = nvlink.ExchangeArea.simulated(nvlink.EXCH_GATHER, m, 1, cuda_device)[0]
    ex_r = nvlink.ExchangeArea.simulated(nvlink.EXCH_REDUCE, n, 1, cuda_device)[0]
    ex_r_small = nvlink.ExchangeArea.simulated(nvlink.EXCH_REDUCE, n // 2, 1, cuda_device)[0]
    bad = [
        lambda: nvlink.lift_dot_allreduce(x, x[:-1], ex_dot),
        lambda: nvlink.lift_dot_allreduce(x, x, ex_dot, out=torch.empty(2, device=cuda_device)),
        lambda: nvlink.lift_dot_allreduce(x, x, ex_g),
        lambda: nvlink.lift_gemv_allgather(A, x, 0, m, ex_g, out=torch.empty(m - 1, device=cuda_device)),
        lambda: nvlink.lift_gemv_allgather(A, x[:-4], 0, m, ex_g),
        lambda: nvlink.lift_gemv_allgather(A, x, 0, m, ex_g, B=A[:-1]),
        lambda: nvlink.lift_gemv_allgather(A, x, 0, 2 * m, ex_g),  # area made for m rows
        lambda: nvlink.lift_atax_reduce(A, x, ex_r, out=torch.empty(n - 4, device=cuda_device)),
        lambda: nvlink.lift_atax_reduce(A, x, ex_r_small),
        lambda: nvlink.lift_atax_reduce(A, x, ex_g),
    ]
    for i, call in enumerate(bad):
        with pytest.raises((ValueError, TypeError)):
            call()
            pytest.fail(f"case {i} accepted")
    y = nvlink.lift_atax_reduce(A, x, ex_r)  # a valid call still runs
    torch.cuda.synchronize()
    ref, mag = oracle.atax(A.cpu().numpy(), x.cpu().numpy())
    assert oracle.within_tol(y.cpu().numpy(), ref, mag)[0]
