"""Multi-process host logic of the sharded path (world_size 2 and 3, gloo, CPU).

The per-rank compute is injected (oracle results rounded to fp32, standing in
for the CUDA kernels, which need a GPU); everything else — partitioning,
padding, the one collective per op, where the result lands — is exactly the
code the GPU path runs.
"""
import os
import socket
import sys

import numpy as np
import pytest
import torch
import torch.distributed as dist
import torch.multiprocessing as mp

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def _free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def _oracle_ops():
    import oracle
    from paper_conf_cgo_steuwerrd17_b200.shard import LocalOps

    def t(a):
        return torch.from_numpy(np.asarray(a, dtype=np.float32))

    def _dot(x, y, out=None):
        return t(np.float32(oracle.dot(x.numpy(), y.numpy())[0])).reshape(())

    def _gemv(A, x, out=None):
        return t(oracle.gemv(A.numpy(), x.numpy())[0])

    def _gesummv(al, A, be, B, x, out=None):
        return t(oracle.gesummv(al, A.numpy(), be, B.numpy(), x.numpy())[0])

    def _atax(A, x, out=None):
        return t(oracle.atax(A.numpy(), x.numpy())[0])

    return LocalOps(dot=_dot, gemv=_gemv, gesummv=_gesummv, atax=_atax)


def _worker(rank, world, port, m, n, q):
    sys.path.insert(0, ROOT)
    try:
        import oracle
        import synth
        from paper_conf_cgo_steuwerrd17_b200 import shard

        dist.init_process_group("gloo", init_method=f"tcp://127.0.0.1:{port}", rank=rank, world_size=world)
        ops = _oracle_ops()
        r0, r1 = shard.partition_rows(m, world, rank)
        A = synth.numpy_matrix_rows(synth.SEED_A, n, r0, r1)  # each rank generates only its rows
        B = synth.numpy_matrix_rows(synth.SEED_B, n, r0, r1)
        x = synth.numpy_uniform(synth.SEED_X, 0, n)
        At, Bt, xt = torch.from_numpy(A), torch.from_numpy(B), torch.from_numpy(x)
        out = {}
        out["gemv"] = shard.gemv(At, xt, m, local=ops).numpy()
        out["gesummv"] = shard.gesummv(1.5, At, 1.2, Bt, xt, m, local=ops).numpy()
        ya = shard.atax(At, xt, dst=0, local=ops)
        out["atax"] = None if ya is None else ya.numpy()
        out["atax_all"] = shard.atax(At, xt, allreduce=True, local=ops).numpy()
        # dot over element slices of length m*n
        N = m * n
        e0, e1 = shard.partition_rows(N, world, rank)
        xd = torch.from_numpy(synth.numpy_uniform(synth.SEED_X, e0, e1 - e0))
        yd = torch.from_numpy(synth.numpy_uniform(synth.SEED_Y, e0, e1 - e0))
        out["dot"] = float(shard.dot(xd, yd, local=ops))
        out["rows"] = (r0, r1)
        q.put((rank, out, None))
        dist.destroy_process_group()
    except Exception as ex:  # pragma: no cover - reported to the parent
        import traceback

        q.put((rank, None, traceback.format_exc()))


@pytest.mark.parametrize("world,m,n", [(2, 64, 48), (2, 37, 20), (3, 50, 16)])
def test_sharded_host_logic_gloo(world, m, n):
    import oracle
    import synth

    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _free_port()
    procs = [ctx.Process(target=_worker, args=(r, world, port, m, n, q)) for r in range(world)]
    for p in procs:
        p.start()
    res = {}
    for _ in range(world):
        rank, out, err = q.get(timeout=180)
        assert err is None, err
        res[rank] = out
    for p in procs:
        p.join(timeout=60)
        assert p.exitcode == 0

    A = synth.numpy_matrix_rows(synth.SEED_A, n, 0, m)
    B = synth.numpy_matrix_rows(synth.SEED_B, n, 0, m)
    x = synth.numpy_uniform(synth.SEED_X, 0, n)
    # partition covers [0, m) exactly once
    rows = sorted(res[r]["rows"] for r in range(world))
    assert rows[0][0] == 0 and rows[-1][1] == m and all(a[1] == b[0] for a, b in zip(rows, rows[1:]))
    ref_gemv = oracle.gemv(A, x)[0].astype(np.float32)
    ref_ges = oracle.gesummv(1.5, A, 1.2, B, x)[0].astype(np.float32)
    for r in range(world):
        # rows are independent: the gathered y is exactly the unsharded one
        assert np.array_equal(res[r]["gemv"], ref_gemv)
        assert np.array_equal(res[r]["gesummv"], ref_ges)
    # ATAX: sum of per-shard partials equals the full result within fp32 rounding of the partials
    ref_atax, mag = oracle.atax(A, x)
    assert res[0]["atax"] is not None
    for r in range(1, world):
        assert res[r]["atax"] is None
    ok, margin = oracle.within_tol(res[0]["atax"], ref_atax, mag)
    assert ok, margin
    for r in range(world):
        assert np.array_equal(res[r]["atax_all"], res[0]["atax"])
    xs = synth.numpy_uniform(synth.SEED_X, 0, m * n)
    ys = synth.numpy_uniform(synth.SEED_Y, 0, m * n)
    ref_dot, dmag = oracle.dot(xs, ys)
    for r in range(world):
        ok, margin = oracle.within_tol([res[r]["dot"]], [ref_dot], [dmag])
        assert ok, margin


def _selfcheck_worker(rank, world, port, fail_rank, q):
    sys.path.insert(0, ROOT)
    try:
        from paper_conf_cgo_steuwerrd17_b200 import shard

        dist.init_process_group("gloo", init_method=f"tcp://127.0.0.1:{port}", rank=rank, world_size=world)
        ops = _oracle_ops()
        shard.cuda_ops = lambda: ops  # per-rank compute without a GPU
        # stand-ins for the fused ops: the collective path itself (so they agree) ...
        shard.dot_fused = lambda x, y, fg, out=None: shard.dot(x, y, fg.group)
        shard.gemv_fused = lambda A, x, m, fg, out=None: shard.gemv(A, x, m, fg.group)
        shard.gesummv_fused = lambda a, A, b, B, x, m, fg, out=None: shard.gesummv(a, A, b, B, x, m, fg.group)
        shard.atax_fused = lambda A, x, fg, dst=0, allreduce=False, out=None: shard.atax(A, x, fg.group, dst, allreduce)
        if rank == fail_rank:  # ... except one op on one rank, which returns wrong bits
            shard.gesummv_fused = lambda a, A, b, B, x, m, fg, out=None: shard.gesummv(a, A, b, B, x, m, fg.group) + 1
        why = shard.fused_self_check(shard.FusedGroup(), torch.device("cpu"))
        q.put((rank, why, None))
        dist.destroy_process_group()
    except Exception:  # pragma: no cover - reported to the parent
        import traceback

        q.put((rank, None, traceback.format_exc()))


@pytest.mark.parametrize("fail_rank", [-1, 1])
def test_fused_self_check_verdict_gloo(fail_rank):
    """bench.py --collectives auto: every rank reaches the same verdict; a
    mismatch on one rank sends all ranks back to the NCCL path."""
    world = 2
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _free_port()
    procs = [ctx.Process(target=_selfcheck_worker, args=(r, world, port, fail_rank, q)) for r in range(world)]
    for p in procs:
        p.start()
    res = {}
    for _ in range(world):
        rank, why, err = q.get(timeout=180)
        assert err is None, err
        res[rank] = why
    for p in procs:
        p.join(timeout=60)
    if fail_rank < 0:
        assert res == {0: None, 1: None}
    else:
        assert res[fail_rank] == "gesummv all-gather differs"
        assert res[1 - fail_rank] == "failed on another rank"


def test_partition_rows_properties():
    from paper_conf_cgo_steuwerrd17_b200.shard import partition_rows, shard_sizes

    for m in (0, 1, 7, 64, 4096, 8192, 65536, 1 << 31):
        for g in (1, 2, 3, 4, 8):
            parts = [partition_rows(m, g, r) for r in range(g)]
            assert parts[0][0] == 0 and parts[-1][1] == m
            assert all(a[1] == b[0] for a, b in zip(parts, parts[1:]))
            sz = shard_sizes(m, g)
            assert max(sz) - min(sz) <= 1
    with pytest.raises(ValueError):
        partition_rows(5, 2, 2)
