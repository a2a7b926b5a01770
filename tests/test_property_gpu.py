"""Property-based parity (hypothesis): random shapes, base offsets (alignment),
scalars and value distributions; every op must meet the north_star tolerance
against the oracle, and structural invariants must hold bitwise."""
import numpy as np
import pytest
import torch
from hypothesis import HealthCheck, given, settings
from hypothesis import strategies as st

import oracle
import synth
import paper_conf_cgo_steuwerrd17_b200 as lift

pytestmark = pytest.mark.gpu
SETTINGS = settings(max_examples=30, deadline=None, suppress_health_check=list(HealthCheck), derandomize=True)

shapes = st.tuples(st.integers(0, 300), st.integers(0, 3000))
offsets = st.integers(0, 3)
seeds = st.integers(0, 10_000)
dists = st.sampled_from(["sym", "pos", "wide"])
scalars = st.sampled_from([0.0, 1.0, -1.0, 0.5, 1.5, 1.2, -3.25, 1e-3])


def dev(a, off=0):
    """Copy to the GPU at a base offset of `off` floats (alignment coverage)."""
    flat = np.ascontiguousarray(a, dtype=np.float32).ravel()
    buf = torch.empty(flat.size + off, dtype=torch.float32, device="cuda")
    t = buf[off:]
    t.copy_(torch.from_numpy(flat))
    return t.view(a.shape) if np.ndim(a) else t


def gen(seed, shape, dist):
    """"sym" U[-1,1), "pos" U[0,1) (both on a 2^-23 / 2^-24 grid), or "wide": full
    24-bit significands over binary exponents -140..20 (subnormals included),
    random signs — rounding behaviour the grid inputs never exercise."""
    cnt = int(np.prod(shape)) if len(shape) else 1
    if dist == "wide":
        return synth.numpy_wide(seed, 0, cnt).reshape(shape)
    return synth.numpy_uniform(seed, 0, cnt, dist).reshape(shape)


def ok(got, ref, mag):
    good, margin = oracle.within_tol(got, ref, mag)
    assert good, margin


@SETTINGS
@given(n=st.integers(0, 200_000), off=offsets, seed=seeds, dist=dists)
def test_dot_property(cuda_device, n, off, seed, dist):
    x, y = gen(seed, (n,), dist), gen(seed + 1, (n,), dist)
    got = lift.lift_dot(dev(x, off), dev(y, (off * 3) % 4)).item()
    ok([got], *[[v] for v in oracle.dot(x, y)])


@SETTINGS
@given(mn=shapes, off=offsets, seed=seeds, dist=dists)
def test_gemv_property(cuda_device, mn, off, seed, dist):
    m, n = mn
    A, x = gen(seed, (m, n), dist), gen(seed + 1, (n,), dist)
    got = lift.lift_gemv(dev(A, off), dev(x, off)).cpu().numpy()
    ok(got, *oracle.gemv(A, x))


@SETTINGS
@given(mn=shapes, off=offsets, seed=seeds, al=scalars, be=scalars, dist=dists)
def test_gesummv_property(cuda_device, mn, off, seed, al, be, dist):
    m, n = mn
    A, B, x = gen(seed, (m, n), dist), gen(seed + 1, (m, n), dist), gen(seed + 2, (n,), dist)
    got = lift.lift_gesummv(al, dev(A, off), be, dev(B, off), dev(x, off)).cpu().numpy()
    ok(got, *oracle.gesummv(al, A, be, B, x))


@SETTINGS
@given(mn=shapes, off=offsets, seed=seeds, algo=st.sampled_from(["auto", "twopass", "fused"]), dist=dists)
def test_atax_property(cuda_device, mn, off, seed, algo, dist):
    m, n = mn
    if algo == "fused" and (off != 0 or n % 4 or n > 16384 or m == 0 or n == 0):
        algo = "auto"
    A, x = gen(seed, (m, n), dist), gen(seed + 1, (n,), dist)
    got = lift.lift_atax(dev(A, off), dev(x, off), algo=algo).cpu().numpy()
    ok(got, *oracle.atax(A, x))


@SETTINGS
@given(mn=shapes, seed=seeds, rows=st.data())
def test_gemv_row_shard_bitwise(cuda_device, mn, seed, rows):
    m, n = mn
    if m == 0:
        return
    A, x = dev(gen(seed, (m, n), "sym")), dev(gen(seed + 1, (n,), "sym"))
    full = lift.lift_gemv(A, x)
    r0 = rows.draw(st.integers(0, m - 1))
    r1 = rows.draw(st.integers(r0 + 1, m))
    assert torch.equal(lift.lift_gemv(A[r0:r1].contiguous(), x), full[r0:r1])


@SETTINGS
@given(n=st.integers(0, 100_000), seed=seeds, contract=st.booleans())
def test_listing1_property_bitwise(cuda_device, n, seed, contract):
    x, y = gen(seed, (n,), "sym"), gen(seed + 1, (n,), "sym")
    got = lift.lift_dot_listing1(dev(x), dev(y), contract=contract).item()
    ref = oracle.dot_listing1_f32(x, y, use_fma=contract)
    assert np.float32(got).view(np.uint32) == np.float32(ref).view(np.uint32)
