"""The production multi-GPU path, executed on the one GPU this build has:
``init_process_group("nccl")`` at world size 1, the NCCL-backed ``shard.*``
ops, and the fused collectives over torch SYMMETRIC MEMORY (the transport a
multi-GPU run uses; the other GPU tests use simulated ranks or CUDA IPC),
each against the fp64 oracle; then a CUDA graph of fused calls replayed
several times (the exchange epoch lives on the device, so replays need no
host-side counter).  Runs in a subprocess: a process group is global state.
"""
import os
import socket
import subprocess
import sys

import pytest

pytestmark = [pytest.mark.gpu, pytest.mark.timeout(600)]
ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def _port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def test_nccl_and_symmetric_memory_world1(cuda_device):
    env = dict(os.environ, MASTER_ADDR="127.0.0.1", MASTER_PORT=str(_port()), WORLD_SIZE="1", RANK="0",
               LOCAL_RANK="0", PYTHONPATH=ROOT)
    r = subprocess.run([sys.executable, os.path.abspath(__file__)], env=env, cwd=ROOT, capture_output=True,
                       text=True, timeout=540)
    assert r.returncode == 0, (r.stdout[-3000:], r.stderr[-4000:])
    assert "world1 ok" in r.stdout, r.stdout[-3000:]
    assert "transport symm" in r.stdout, r.stdout[-3000:]


def _child():
    import numpy as np
    import torch
    import torch.distributed as dist

    import oracle
    import synth
    from paper_conf_cgo_steuwerrd17_b200 import shard

    dev = torch.device("cuda", 0)
    torch.cuda.set_device(dev)
    dist.init_process_group("nccl", device_id=dev)
    assert dist.get_backend() == "nccl" and dist.get_world_size() == 1

    def ok(got, ref, mag, what):
        good, margin = oracle.within_tol(np.atleast_1d(got), np.atleast_1d(ref), np.atleast_1d(mag))
        assert good, (what, margin)

    nd, m, n = (1 << 20) + 3, 1000, 4096
    x = synth.torch_uniform(synth.SEED_X, 0, nd, device=dev)
    y = synth.torch_uniform(synth.SEED_Y, 0, nd, device=dev)
    A = synth.torch_matrix_rows(synth.SEED_A, n, 0, m, device=dev)
    B = synth.torch_matrix_rows(synth.SEED_B, n, 0, m, device=dev)
    xv = synth.torch_uniform(7, 0, n, device=dev)
    xn, yn, An, Bn, xvn = (t.cpu().numpy() for t in (x, y, A, B, xv))
    rd, rg, rs, ra = oracle.dot(xn, yn), oracle.gemv(An, xvn), oracle.gesummv(1.5, An, 1.2, Bn, xvn), \
        oracle.atax(An, xvn)

    # ---- NCCL collectives (one per op) ----
    ok(shard.dot(x, y).item(), *rd, "nccl dot")
    ok(shard.gemv(A, xv, m).cpu().numpy(), *rg, "nccl gemv")
    ok(shard.gesummv(1.5, A, 1.2, B, xv, m).cpu().numpy(), *rs, "nccl gesummv")
    ok(shard.atax(A, xv, dst=0).cpu().numpy(), *ra, "nccl atax")
    ok(shard.atax(A, xv, allreduce=True).cpu().numpy(), *ra, "nccl atax allreduce")

    # ---- the collectives fused into the kernels, over torch symmetric memory ----
    fg = shard.FusedGroup(transport="symm")
    assert shard.fused_self_check(fg, dev) is None
    print("transport symm:", sorted(fg.areas), flush=True)
    outs = dict(d=torch.empty((), device=dev), g=torch.empty(m, device=dev), s=torch.empty(m, device=dev),
                a=torch.empty(n, device=dev))

    def step(xvec):
        shard.dot_fused(x, y, fg, out=outs["d"])
        shard.gemv_fused(A, xvec, m, fg, out=outs["g"])
        shard.gesummv_fused(1.5, A, 1.2, B, xvec, m, fg, out=outs["s"])
        shard.atax_fused(A, xvec, fg, dst=0, out=outs["a"])

    def check(what):
        torch.cuda.synchronize()
        ok(outs["d"].item(), *rd, f"{what} dot")
        ok(outs["g"].cpu().numpy(), *rg, f"{what} gemv")
        ok(outs["s"].cpu().numpy(), *rs, f"{what} gesummv")
        ok(outs["a"].cpu().numpy(), *ra, f"{what} atax")

    s = torch.cuda.Stream()
    with torch.cuda.stream(s):
        for _ in range(3):
            step(xv)
        check("eager")
        # a CUDA graph of fused calls, replayed: each replay is a new epoch on the device
        xg = xv.clone()
        g = torch.cuda.CUDAGraph()
        with torch.cuda.graph(g, stream=s):
            step(xg)
        for k in range(4):
            for o in outs.values():
                o.fill_(float("nan"))
            g.replay()
            check(f"graph replay {k}")
    dist.destroy_process_group()
    print("world1 ok", flush=True)


if __name__ == "__main__":
    _child()
