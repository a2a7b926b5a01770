"""Chains of the library's ops on one stream, each op reading the previous
op's output, with no host synchronisation in between — eagerly and replayed
from a CUDA graph.

Every kernel is launched with programmatic dependent launch (include/lift.h:
a kernel may be scheduled while its predecessor drains and waits with
griddepcontrol.wait before touching memory).  A kernel that read global
memory before that wait would see its input half-written: every output buffer
is filled with NaN beforehand and every stage is checked against the oracle
applied to the GPU's own input for that stage, so a premature read shows up as
NaN or as a wrong value.
"""
import numpy as np
import pytest
import torch

import oracle
import synth
import paper_conf_cgo_steuwerrd17_b200 as lift

pytestmark = [pytest.mark.gpu, pytest.mark.timeout(600)]

N = 4096
ALPHA, BETA = 1.5, -0.5


@pytest.fixture(scope="module")
def mats(cuda_device):
    # entries U[-1/64, 1/64): every stage keeps its values O(1)
    return [synth.torch_matrix_rows(synth.SEED_A + 10 * k, N, 0, N, device=cuda_device) / 64 for k in range(4)]


def chain(A, x, outs):
    """One pass: 13 ops (17 kernels), each consuming the previous results."""
    A1, A2, A3, A4 = A
    lift.lift_gemv(A1, x, out=outs["y1"])
    lift.lift_atax(A2, outs["y1"], out=outs["y2"], algo="fused")
    lift.lift_gesummv(ALPHA, A3, BETA, A4, outs["y2"], out=outs["y3"])
    outs["y4"].copy_(outs["y3"])  # the SGEMV's y is read (beta != 0) and updated in place
    lift.lift_sgemv(1.0, A1, outs["y3"], beta=0.25, y=outs["y4"], trans=True)
    lift.lift_atax(A2, outs["y4"], out=outs["y5"], algo="twopass")
    lift.lift_dot(outs["y5"], outs["y1"], out=outs["s6"])
    lift.lift_partial_dot(outs["y5"], outs["y3"], out=outs["z7"])
    lift.lift_gemv(A3, outs["y5"], out=outs["y8"])
    lift.lift_dot_listing1(outs["y8"], outs["y8"], out=outs["s9"])
    # a MATRIX produced by the kernel right before: the dependent GEMV / fused ATAX
    # blocks prefetch their first rows into L2 before griddepcontrol.wait, while the
    # producer (which lets its dependents launch at its start) may still be writing
    # them; only the loads after the wait may deliver data (common.cuh)
    lift.lift_gemv(A3, outs["y8"], out=outs["y10"])
    lift.lift_gemv(outs["y10"].view(16, 256), outs["y1"][:256], out=outs["y11"])
    lift.lift_gemv(A4, outs["y10"], out=outs["y12"])
    lift.lift_atax(outs["y12"].view(16, 256), outs["y1"][:256], out=outs["y13"], algo="fused")


def fresh_outputs(device):
    nan = float("nan")
    o = {k: torch.full((N,), nan, device=device) for k in ("y1", "y2", "y3", "y4", "y5", "y8", "y10", "y12")}
    o["y11"] = torch.full((16,), nan, device=device)
    o["y13"] = torch.full((256,), nan, device=device)
    o["s6"] = torch.full((), nan, device=device)
    o["s9"] = torch.full((), nan, device=device)
    o["z7"] = torch.full((N // 128,), nan, device=device)
    return o


def check_chain(A, x, outs):
    """Each stage against the oracle on the GPU's own input to that stage."""
    h = {k: v.cpu().numpy() for k, v in outs.items()}
    A1, A2, A3, A4 = (a.cpu().numpy() for a in A)
    xs = x.cpu().numpy()
    y3_in = h["y3"]

    def ok(name, got, ref_mag):
        ref, mag = ref_mag
        assert np.all(np.isfinite(got)), f"{name}: non-finite values (a read before the producer finished?)"
        good, margin = oracle.within_tol(np.atleast_1d(got), np.atleast_1d(ref), np.atleast_1d(mag))
        assert good, f"{name}: margin {margin:.3g}"

    ok("gemv", h["y1"], oracle.gemv(A1, xs))
    ok("atax fused", h["y2"], oracle.atax(A2, h["y1"]))
    ok("gesummv", h["y3"], oracle.gesummv(ALPHA, A3, BETA, A4, h["y2"]))
    ok("sgemv^T", h["y4"], oracle.sgemv(0, 1, N, N, 1.0, A1.ravel(), N, y3_in, 0.25, y3_in))
    ok("atax twopass", h["y5"], oracle.atax(A2, h["y4"]))
    ok("dot", h["s6"], oracle.dot(h["y5"], h["y1"]))
    ok("partial dot", h["z7"], oracle.partial_dot(h["y5"], h["y3"]))
    ok("gemv 2", h["y8"], oracle.gemv(A3, h["y5"]))
    ok("gemv 3", h["y10"], oracle.gemv(A3, h["y8"]))
    ok("gemv of a produced matrix", h["y11"], oracle.gemv(h["y10"].reshape(16, 256), h["y1"][:256]))
    ok("gemv 4", h["y12"], oracle.gemv(A4, h["y10"]))
    ok("atax of a produced matrix", h["y13"], oracle.atax(h["y12"].reshape(16, 256), h["y1"][:256]))
    assert np.float32(h["s9"]).view(np.uint32) == np.float32(oracle.dot_listing1_f32(h["y8"], h["y8"])).view(
        np.uint32), "listing-1 dot differs from the paper-order emulation"


def test_chain_eager(cuda_device, mats):
    xs = [synth.torch_uniform(synth.SEED_X + r, 0, N, device=cuda_device) for r in range(3)]
    outs = [fresh_outputs(cuda_device) for _ in xs]
    torch.cuda.synchronize()
    for x, o in zip(xs, outs):  # three passes back to back, no synchronisation
        chain(mats, x, o)
    torch.cuda.synchronize()
    for x, o in zip(xs, outs):
        check_chain(mats, x, o)


def test_chain_graph(cuda_device, mats):
    xs = [synth.torch_uniform(synth.SEED_X + 7 + r, 0, N, device=cuda_device) for r in range(2)]
    outs = [fresh_outputs(cuda_device) for _ in xs]
    s = torch.cuda.Stream()
    s.wait_stream(torch.cuda.current_stream())
    with torch.cuda.stream(s):  # warm-up outside the graph (workspaces on this stream)
        for x, o in zip(xs, outs):
            chain(mats, x, o)
    torch.cuda.synchronize()
    for o in outs:
        for v in o.values():
            v.fill_(float("nan"))
    g = torch.cuda.CUDAGraph()
    with torch.cuda.graph(g, stream=s):
        for x, o in zip(xs, outs):
            chain(mats, x, o)
    for rep in range(2):
        for o in outs:
            for v in o.values():
                v.fill_(float("nan"))
        torch.cuda.synchronize()
        g.replay()
        torch.cuda.synchronize()
        for x, o in zip(xs, outs):
            check_chain(mats, x, o)
