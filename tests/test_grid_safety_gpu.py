"""Grid barriers under SM pressure: never a hang.

The fused ATAX kernels end in a grid barrier (every block waits for every
other block), which needs all blocks resident at once.  A concurrent kernel
holding SMs (tests/cuda/hog.cu: one 160 KiB-shared-memory block per SM,
spinning until released) must therefore either delay the launch (cooperative
launches: the single-block kernel, and the cluster kernel launched cooperative
with its cluster shape) or make the barrier fail cleanly with a CUDA error
after the spin limit (LIFT_SPIN_TIMEOUT_MS) — never hang the GPU.

Each case runs in a subprocess: a trapped kernel ends its CUDA context.
"""
import ctypes
import os
import subprocess
import sys
import threading
import time

import pytest

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
FREE_SMS = 8

pytestmark = [pytest.mark.gpu, pytest.mark.timeout(300)]


@pytest.fixture(scope="module")
def hog_so(tmp_path_factory):
    so = str(tmp_path_factory.mktemp("hog") / "libhog.so")
    subprocess.check_call(["nvcc", "-gencode", "arch=compute_100a,code=sm_100a", "-shared", "-Xcompiler", "-fPIC",
                           "-o", so, os.path.join(ROOT, "tests", "cuda", "hog.cu")])
    return so


def run_child(case, so, spin_ms, release_s):
    env = dict(os.environ, LIFT_SPIN_TIMEOUT_MS=str(spin_ms), PYTHONPATH=ROOT)
    t0 = time.time()
    r = subprocess.run([sys.executable, os.path.abspath(__file__), case, so, str(release_s)], env=env,
                       capture_output=True, text=True, timeout=240)
    return r, time.time() - t0


@pytest.mark.parametrize("shape", ["narrow", "wide"])
def test_cooperative_launch_waits_for_sms(hog_so, shape):
    """The library's own launches of the grid-barrier kernels are cooperative:
    with all but 8 SMs held, the kernel waits for the hog to let go (released
    after 4 s, beyond the 2 s spin limit) and then computes the right result."""
    r, _ = run_child(shape, hog_so, 2000, 4.0)
    assert r.returncode == 0, r.stdout + r.stderr
    assert "parity ok" in r.stdout, r.stdout
    waited = float(r.stdout.split("completed after ")[1].split(" s")[0])
    assert waited >= 3.5, r.stdout  # it did wait for the hog


def test_plain_launch_grid_barrier_fails_cleanly(hog_so):
    """A plain launch that cannot be co-resident (the explicit-grid exchange entry
    point; tests run several ranks on one GPU with it) spins in the grid barrier
    only until the spin limit, then traps: the call's stream reports a CUDA error
    within seconds, and the process (the hog still holding SMs) exits normally."""
    r, el = run_child("plain", hog_so, 1500, 30.0)
    assert r.returncode == 0, r.stdout + r.stderr
    assert "failed after" in r.stdout, r.stdout
    failed = float(r.stdout.split("failed after ")[1].split(" s")[0])
    assert 1.0 <= failed < 15.0, r.stdout
    assert el < 60


def test_missing_peer_fails_cleanly(hog_so):
    """A fused collective whose peer never makes the matching call (rank 1 of a
    simulated world of 2 never launches): rank 0's kernel waits for the peer's
    flag only until the spin limit, then traps — a CUDA error, not a hang."""
    r, el = run_child("peer", hog_so, 1500, 0.0)
    assert r.returncode == 0, r.stdout + r.stderr
    assert "failed after" in r.stdout, r.stdout
    failed = float(r.stdout.split("failed after ")[1].split(" s")[0])
    assert 1.0 <= failed < 15.0, r.stdout
    assert el < 60


# --------------------------------------------------------------------- child process
def _peer_child():
    import torch

    import synth
    from paper_conf_cgo_steuwerrd17_b200 import nvlink

    dev = torch.device("cuda", 0)
    n = 1 << 16
    x = synth.torch_uniform(synth.SEED_X, 0, n, device=dev)
    exs = nvlink.ExchangeArea.simulated(nvlink.EXCH_DOT, 0, 2, dev)
    ws = torch.zeros(nvlink.workspace_bytes("dot", 0, n), dtype=torch.uint8, device=dev)
    out = torch.empty((), device=dev)
    torch.cuda.synchronize()
    t1 = time.time()
    try:
        nvlink.lift_dot_allreduce(x, x, exs[0], out=out, workspace=ws)  # rank 1 never calls
        torch.cuda.synchronize()
        print(f"completed after {time.time() - t1:.2f} s (unexpected)", flush=True)
    except Exception as e:  # noqa: BLE001
        print(f"failed after {time.time() - t1:.2f} s: {type(e).__name__}: {str(e)[:200]}", flush=True)
    os._exit(0)


def _child(case, so, release_s):
    if case == "peer":
        _peer_child()
    import torch

    import oracle
    import synth
    import paper_conf_cgo_steuwerrd17_b200 as lift
    from paper_conf_cgo_steuwerrd17_b200 import nvlink

    dev = torch.device("cuda", 0)
    m, n = (8192, 32768) if case == "wide" else (4096, 4096)
    A = synth.torch_matrix_rows(synth.SEED_A, n, 0, m, device=dev)
    x = synth.torch_uniform(synth.SEED_X, 0, n, device=dev)
    if case == "plain":
        ex = nvlink.ExchangeArea.simulated(nvlink.EXCH_REDUCE, n, 1, dev)[0]
        ws = torch.zeros(nvlink.workspace_bytes("atax", m, n), dtype=torch.uint8, device=dev)
        out = torch.empty(n, device=dev)
        sms = torch.cuda.get_device_properties(0).multi_processor_count

        def call():
            return nvlink.lift_atax_reduce(A, x, ex, dst=-1, blocks=sms, out=out, workspace=ws)
    else:
        def call():
            return lift.lift_atax(A, x, algo="fused")
    y = call()  # warm-up: workspaces allocated, result checked below
    torch.cuda.synchronize()
    hog = ctypes.CDLL(so)
    sms = torch.cuda.get_device_properties(0).multi_processor_count
    hs = torch.cuda.Stream()
    assert hog.hog_start(sms - FREE_SMS, 160 * 1024, ctypes.c_ulonglong(int(60e9)),
                         ctypes.c_void_p(hs.cuda_stream)) == 0
    t0 = time.time()
    while hog.hog_started() < sms - FREE_SMS and time.time() - t0 < 10:
        time.sleep(0.01)
    assert hog.hog_started() == sms - FREE_SMS
    timer = threading.Timer(release_s, hog.hog_release)
    timer.start()
    t1 = time.time()
    try:
        y = call()
        torch.cuda.synchronize()
        el = time.time() - t1
        ref, mag = oracle.atax(A.cpu().numpy(), x.cpu().numpy())
        ok, margin = oracle.within_tol(y.cpu().numpy(), ref, mag)
        print(f"completed after {el:.2f} s, parity {'ok' if ok else 'BAD'} margin={margin:.3g}", flush=True)
    except Exception as e:  # noqa: BLE001 — the trapped launch surfaces as a CUDA error
        print(f"failed after {time.time() - t1:.2f} s: {type(e).__name__}: {str(e)[:200]}", flush=True)
    hog.hog_release()
    timer.cancel()
    os._exit(0)  # the context may be dead: skip interpreter teardown of CUDA state


if __name__ == "__main__":
    _child(sys.argv[1], sys.argv[2], float(sys.argv[3]))
