"""Pins for the fp64 CPU oracle (oracle/) against things other than itself.

Each test checks the oracle against what the paper or the mathematics fixes:
exact rational brute force (fractions.Fraction), closed forms, invariants, the
paper's printed index formulas (tests/golden/, each with its citation) and
hand-derived fp32 results of Listing 1.  A plausible slip in the oracle — a
dropped term, a wrong sign or index, a transposed operand, a wrong chunk —
fails at least one of them.  No test here touches the CUDA path.
"""
from fractions import Fraction

import numpy as np
import pytest

import oracle
import synth
from conftest import golden

EPS64 = 2.0 ** -53


# ---------------------------------------------------------------------------
# exact references (Fraction) — independent of the oracle's C loops
# ---------------------------------------------------------------------------

def F(v):
    return Fraction(float(v))


def exact_matvec(A, x):
    """Exact rational y = A x (lists of Fractions)."""
    m, n = A.shape
    return [sum((F(A[i, j]) * F(x[j]) for j in range(n)), Fraction(0)) for i in range(m)]


def exact_abs_matvec(A, x):
    m, n = A.shape
    return [sum((abs(F(A[i, j]) * F(x[j])) for j in range(n)), Fraction(0)) for i in range(m)]


def rand_f32(seed, shape, dist="sym"):
    cnt = int(np.prod(shape))
    return synth.numpy_uniform(seed, 0, cnt, dist).reshape(shape)


def assert_close_exact(got, exact, n_terms, mag):
    """|got - exact| <= n * 2^-53 * mag  (fp64 summation bound)."""
    for g, e, mg in zip(np.atleast_1d(got), exact, np.atleast_1d(mag)):
        bound = (n_terms + 1) * EPS64 * float(mg) + 1e-300
        assert abs(Fraction(float(g)) - e) <= Fraction(bound), (g, float(e), bound)


# ---------------------------------------------------------------------------
# dot — L285
# ---------------------------------------------------------------------------

@pytest.mark.parametrize("n", [0, 1, 2, 3, 7, 31, 64])
@pytest.mark.parametrize("seed", [0, 5])
def test_dot_bruteforce_fraction(n, seed):
    x = rand_f32(seed, (n,))
    y = rand_f32(seed + 100, (n,))
    s, mag = oracle.dot(x, y)
    exact = sum((F(a) * F(b) for a, b in zip(x, y)), Fraction(0))
    exact_mag = sum((abs(F(a) * F(b)) for a, b in zip(x, y)), Fraction(0))
    assert_close_exact([s], [exact], n, [mag])
    assert abs(Fraction(mag) - exact_mag) <= Fraction((n + 1) * EPS64 * float(exact_mag) + 1e-300)


@pytest.mark.parametrize("n", [1, 5, 33, 64])
def test_dot_chunked_bruteforce_and_extremes(n):
    # the all-core dot (reading R23): Fraction brute force within the fp64 bound, and
    # its two extreme groupings ARE the plain left fold — one chunk (the fold itself)
    # and one element per chunk (exact products folded in order)
    x, y = rand_f32(3, (n,)), rand_f32(4, (n,))
    exact = sum((F(a) * F(b) for a, b in zip(x, y)), Fraction(0))
    exact_mag = sum((abs(F(a) * F(b)) for a, b in zip(x, y)), Fraction(0))
    s1, m1 = oracle.dot(x, y)
    for chunks in (1, 2, 3, n):
        s, mag = oracle.dot_chunked(x, y, chunks=chunks, threads=3)
        assert_close_exact([s], [exact], n, [mag])
        assert_close_exact([mag], [exact_mag], n, [mag])
    assert oracle.dot_chunked(x, y, chunks=1)[0] == s1
    assert oracle.dot_chunked(x, y, chunks=n)[0] == s1
    # wide-range data, where fp64 association matters: still exactly the left fold at
    # the two extremes (so the chunk sums are combined in chunk order)
    xw, yw = synth.numpy_wide(5, 0, 4096, -60, 60), synth.numpy_wide(6, 0, 4096, -60, 60)
    sw, _ = oracle.dot(xw, yw)
    assert sw != oracle.dot(xw[::-1], yw[::-1])[0]  # the data does separate orders
    assert oracle.dot_chunked(xw, yw, chunks=1)[0] == sw
    assert oracle.dot_chunked(xw, yw, chunks=4096, threads=4)[0] == sw


def test_dot_chunked_thread_invariant_and_close():
    n = (1 << 22) + 17
    x, y = rand_f32(0, (n,)), rand_f32(1, (n,))
    ref = oracle.dot_chunked(x, y, chunks=256, threads=1)
    for th in (2, 5, 16):
        assert oracle.dot_chunked(x, y, chunks=256, threads=th) == ref
    s, mag = oracle.dot(x, y)
    assert abs(ref[0] - s) <= 1e-12 * mag and ref[1] == pytest.approx(mag, rel=1e-12)


def test_dot_empty_is_zero():
    # reduceSeq(z=0, f, []) = z  (L320)
    s, mag = oracle.dot(np.zeros(0, np.float32), np.zeros(0, np.float32))
    assert s == 0.0 and mag == 0.0


def test_dot_ones_closed_form():
    for n in (1, 128, 4097, 1 << 20):
        s, _ = oracle.dot(np.ones(n, np.float32), np.ones(n, np.float32))
        assert s == float(n)


def test_dot_ramp_closed_form():
    g = golden("closed_forms.json")["dot_ramp"]
    n = g["n"]
    x = np.arange(n, dtype=np.float32)  # exact for n <= 2^24
    s, mag = oracle.dot(x, np.ones(n, np.float32))
    assert s == float(g["expected"]) == n * (n - 1) // 2
    assert mag == s


@pytest.mark.parametrize("n,a,d,b,e", [(1 << 17, 3.0, 2.0, -5.0, 1.0), (1000, -7.0, -3.0, 2.0, 5.0)])
def test_dot_two_ramps_closed_form(n, a, d, b, e):
    i = np.arange(n, dtype=np.float64)
    x = (a + i * d).astype(np.float32)
    y = (b + i * e).astype(np.float32)
    assert np.all(x == a + i * d) and np.all(y == b + i * e)  # exactly representable
    s, _ = oracle.dot(x, y)
    N = n
    expected = N * a * b + (a * e + b * d) * (N * (N - 1) // 2) + d * e * ((N - 1) * N * (2 * N - 1) // 6)
    assert s == expected


def test_dot_sign_and_symmetry():
    x = rand_f32(11, (4099,))
    y = rand_f32(12, (4099,))
    sxx, _ = oracle.dot(x, x)
    assert sxx > 0
    assert oracle.dot(x, y)[0] == oracle.dot(y, x)[0]
    # negating one operand negates the result exactly
    assert oracle.dot(-x, y)[0] == -oracle.dot(x, y)[0]


# ---------------------------------------------------------------------------
# GEMV — Table 1
# ---------------------------------------------------------------------------

@pytest.mark.parametrize("m,n", [(1, 1), (3, 5), (7, 2), (16, 13), (5, 16)])
def test_gemv_bruteforce_fraction(m, n):
    A = rand_f32(2, (m, n))
    x = rand_f32(0, (n,))
    y, mag = oracle.gemv(A, x)
    assert_close_exact(y, exact_matvec(A, x), n, mag)
    assert_close_exact(mag, exact_abs_matvec(A, x), n, mag)


def test_gemv_ones_closed_form():
    for m, n in ((4, 4096), (3, 8192), (2, 32768), (5, 3)):
        y, mag = oracle.gemv(np.ones((m, n), np.float32), np.ones(n, np.float32))
        assert np.all(y == n) and np.all(mag == n)


def test_gemv_identity_and_hadamard():
    n = 64
    x = rand_f32(0, (n,))
    y, _ = oracle.gemv(np.eye(n, dtype=np.float32), x)
    assert np.array_equal(y, x.astype(np.float64))
    H = synth.hadamard(n)
    for k in (0, 1, 37, 63):
        e = np.zeros(n, np.float32)
        e[k] = 1
        yk, _ = oracle.gemv(H, e)
        assert np.array_equal(yk, H[:, k].astype(np.float64))
    y1, _ = oracle.gemv(H, np.ones(n, np.float32))
    ref = np.zeros(n)
    ref[0] = n
    assert np.array_equal(y1, ref)


def test_gemv_rows_equal_dot_oracle():
    # y_i = dot(A_i, x): same fold order in both oracle functions
    A = rand_f32(2, (9, 1001))
    x = rand_f32(0, (1001,))
    y, mag = oracle.gemv(A, x)
    for i in range(9):
        s, mg = oracle.dot(A[i], x)
        assert y[i] == s and mag[i] == mg


def test_gemv_thread_count_invariant():
    A = rand_f32(2, (97, 300))
    x = rand_f32(0, (300,))
    y1, m1 = oracle.gemv(A, x, threads=1)
    y8, m8 = oracle.gemv(A, x, threads=8)
    assert np.array_equal(y1, y8) and np.array_equal(m1, m8)


# ---------------------------------------------------------------------------
# GESUMMV — Table 1, reading A9
# ---------------------------------------------------------------------------

@pytest.mark.parametrize("alpha,beta", [(1.5, 1.2), (-0.75, 3.0), (0.0, 1.0), (1.0, 0.0), (-1.0, -1.0)])
def test_gesummv_bruteforce_fraction(alpha, beta):
    m, n = 6, 11
    A = rand_f32(2, (m, n))
    B = rand_f32(3, (m, n))
    x = rand_f32(0, (n,))
    y, mag = oracle.gesummv(alpha, A, beta, B, x)
    a32, b32 = F(np.float32(alpha)), F(np.float32(beta))  # reading A22: fp32 scalars
    ya, yb = exact_matvec(A, x), exact_matvec(B, x)
    exact = [a32 * p + b32 * q for p, q in zip(ya, yb)]
    assert_close_exact(y, exact, 2 * n + 2, mag)
    ma, mb = exact_abs_matvec(A, x), exact_abs_matvec(B, x)
    exact_mag = [abs(a32) * p + abs(b32) * q for p, q in zip(ma, mb)]
    assert_close_exact(mag, exact_mag, 2 * n + 2, mag)


def test_gesummv_alpha_is_fp32_not_decimal():
    # (double)1.2f = 1.2000000476837158 (reading A22)
    A = np.ones((1, 4), np.float32)
    B = np.zeros((1, 4), np.float32)
    y, _ = oracle.gesummv(1.2, A, 0.0, B, np.ones(4, np.float32))
    assert y[0] == 4 * float(np.float32(1.2)) and y[0] != 4 * 1.2


def test_gesummv_linearity_exact():
    # integer data |v| <= 8, n <= 64, power-of-two alpha/beta: every fp64 op exact
    m, n = 12, 64
    A = synth.small_ints(21, m * n, 8).reshape(m, n)
    B = synth.small_ints(22, m * n, 8).reshape(m, n)
    x = synth.small_ints(23, n, 8)
    g10, _ = oracle.gesummv(1.0, A, 0.0, B, x)
    g01, _ = oracle.gesummv(0.0, A, 1.0, B, x)
    for al, be in ((2.0, 0.5), (-4.0, 0.25), (0.125, -8.0)):
        g, _ = oracle.gesummv(al, A, be, B, x)
        assert np.array_equal(g, al * g10 + be * g01)
    # B = A  =>  (alpha + beta) * gemv
    gA, _ = oracle.gemv(A, x)
    g, _ = oracle.gesummv(2.0, A, 4.0, A, x)
    assert np.array_equal(g, 6.0 * gA)
    # beta = 0 => alpha * gemv ; alpha=beta=0 => 0
    g, _ = oracle.gesummv(0.5, A, 0.0, B, x)
    assert np.array_equal(g, 0.5 * gA)
    g, _ = oracle.gesummv(0.0, A, 0.0, B, x)
    assert np.all(g == 0)


def test_gesummv_ones():
    m, n = 3, 8192
    y, _ = oracle.gesummv(1.5, np.ones((m, n), np.float32), 1.25, np.ones((m, n), np.float32),
                          np.ones(n, np.float32))
    assert np.all(y == 2.75 * n)


# ---------------------------------------------------------------------------
# ATAX — Table 1; transpose index Fig. 6 (L796-798)
# ---------------------------------------------------------------------------

def _eval_index(expr, **env):
    return eval(expr, {"__builtins__": {}}, env)  # noqa: S307 (fixture we wrote)


def test_fig6_transpose_index_simplifies():
    g = golden("fig6_transpose_index.json")
    for M, N in ((3, 5), (4, 4), (7, 2)):
        for wg_id in range(N):
            for l_id in range(M):
                v1 = _eval_index(g["line1"], wg_id=wg_id, l_id=l_id, M=M, N=N)
                v2 = _eval_index(g["line2"], wg_id=wg_id, l_id=l_id, M=M, N=N)
                v3 = _eval_index(g["line3"], wg_id=wg_id, l_id=l_id, M=M, N=N)
                assert v1 == v2 == v3


def transpose_via_fig6(A):
    """A^T built with the paper's simplified transpose index (Fig. 6 line 3)."""
    M, N = A.shape  # M rows of length N (row-major, reading A10)
    flat = A.ravel()
    g = golden("fig6_transpose_index.json")
    out = np.empty((N, M), np.float32)
    for wg_id in range(N):
        for l_id in range(M):
            out[wg_id, l_id] = flat[_eval_index(g["line3"], wg_id=wg_id, l_id=l_id, M=M, N=N)]
    return out


@pytest.mark.parametrize("m,n", [(1, 1), (5, 3), (3, 7), (16, 16), (32, 9)])
def test_atax_equals_AtA_x_exact(m, n):
    # integer entries |a| <= 8, |x| <= 8: every intermediate is an integer < 2^53
    A = synth.small_ints(31 + m, m * n, 8).reshape(m, n)
    x = synth.small_ints(32 + n, n, 8)
    y, mag = oracle.atax(A, x)
    At = transpose_via_fig6(A)
    assert np.array_equal(At, A.T)
    AtA = [[sum(int(At[i, k]) * int(A[k, j]) for k in range(m)) for j in range(n)] for i in range(n)]
    ref = [sum(AtA[i][j] * int(x[j]) for j in range(n)) for i in range(n)]
    assert np.array_equal(y, np.array(ref, np.float64))
    # mag = |A|^T (|A| |x|)
    absA = np.abs(A).astype(np.int64)
    mref = absA.T @ (absA @ np.abs(x).astype(np.int64))
    assert np.array_equal(mag, mref.astype(np.float64))


@pytest.mark.parametrize("m,n", [(4, 6), (9, 5)])
def test_atax_bruteforce_fraction_random(m, n):
    A = rand_f32(2, (m, n))
    x = rand_f32(0, (n,))
    y, mag = oracle.atax(A, x)
    t = exact_matvec(A, x)  # exact t (the oracle keeps t in fp64: small extra rounding)
    At = transpose_via_fig6(A)
    exact = [sum((F(At[j, i]) * t[i] for i in range(m)), Fraction(0)) for j in range(n)]
    assert_close_exact(y, exact, m * n + m, mag)


def test_atax_hadamard_identity_permutation():
    n = 256
    H = synth.hadamard(n)
    x = synth.small_ints(41, n, 1023)
    y, _ = oracle.atax(H, x)
    assert np.array_equal(y, n * x.astype(np.float64))  # H^T H = n I
    y, _ = oracle.atax(np.eye(n, dtype=np.float32), x)
    assert np.array_equal(y, x.astype(np.float64))
    perm = np.random.RandomState(0).permutation(n)
    P = np.eye(n, dtype=np.float32)[perm]
    y, _ = oracle.atax(P, x)
    assert np.array_equal(y, x.astype(np.float64))


def test_atax_thread_count_invariant():
    A = rand_f32(2, (50, 77))
    x = rand_f32(0, (77,))
    y1, m1 = oracle.atax(A, x, threads=1)
    y7, m7 = oracle.atax(A, x, threads=7)
    assert np.array_equal(y1, y7) and np.array_equal(m1, m7)


def test_atax_row_shards_sum_to_full():
    # sum over row blocks of A_r^T (A_r x) = A^T (A x)   (north_star sharding)
    A = synth.small_ints(51, 40 * 24, 8).reshape(40, 24)
    x = synth.small_ints(52, 24, 8)
    full, _ = oracle.atax(A, x)
    parts = sum(oracle.atax(A[r0:r1], x)[0] for r0, r1 in ((0, 13), (13, 27), (27, 40)))
    assert np.array_equal(full, parts)


# ---------------------------------------------------------------------------
# partialDot — Listing 1 (L391-401), Fig. 5 (L817), Fig. 7 (L948-981)
# ---------------------------------------------------------------------------

def test_partial_dot_chunks_follow_fig5_index():
    g = golden("fig5_dot_index.json")
    n = 128 * 5
    y = rand_f32(1, (n,))
    for j in (0, 1, 127, 128, 300, n - 1):
        e = np.zeros(n, np.float32)
        e[j] = 1
        z, _ = oracle.partial_dot(e, y, chunk=g["chunk"])
        # the work group whose generated index hits j
        owner = [wg for wg in range(n // 128) for l in range(g["ranges"]["l_id"])
                 for i in range(g["ranges"]["i"]) if _eval_index(g["index"], l_id=l, wg_id=wg, i=i) == j]
        assert len(owner) == 1
        ref = np.zeros(n // 128)
        ref[owner[0]] = y[j]
        assert np.array_equal(z, ref)


def test_partial_dot_sums_to_dot_and_drops_tail():
    n = 128 * 7 + 5  # ragged: Fig. 7 forms only N/128 groups (L954)
    x = rand_f32(0, (n,))
    y = rand_f32(1, (n,))
    z, mag = oracle.partial_dot(x, y)
    assert z.size == 7
    s, _ = oracle.dot(x[:128 * 7], y[:128 * 7])
    assert abs(z.sum() - s) <= 1e-12 * mag.sum()
    for k in range(7):
        exact = sum((F(a) * F(b) for a, b in zip(x[128 * k:128 * k + 128], y[128 * k:128 * k + 128])), Fraction(0))
        assert_close_exact([z[k]], [exact], 128, [mag[k]])
        exact_mag = sum((abs(F(a) * F(b)) for a, b in zip(x[128 * k:128 * k + 128], y[128 * k:128 * k + 128])),
                        Fraction(0))
        assert_close_exact([mag[k]], [exact_mag], 128, [mag[k]])


@pytest.mark.parametrize("use_fma", [True, False])
def test_listing1_fp32_hand_derived(use_fma):
    g = golden("listing1_fp32_order.json")
    for case in g["cases"]:
        x = np.zeros(128, np.float32)
        y = np.zeros(128, np.float32)
        for k, v in case["x"].items():
            x[int(k)] = v
        if "y_all" in case:
            y[:] = case["y_all"]
        else:
            for k, v in case["y"].items():
                y[int(k)] = v
        z = oracle.partial_dot_listing1_f32(x, y, use_fma=use_fma)
        want = case["expected_fma"] if use_fma else case["expected_nofma"]
        assert z.shape == (1,) and float(z[0]) == want, (case["name"], float(z[0]), want)


def test_listing1_fp32_integer_exact():
    # integer data with |partial sums| < 2^24: any order is exact in fp32
    n = 128 * 9
    x = synth.small_ints(61, n, 30)
    y = synth.small_ints(62, n, 30)
    for fma in (True, False):
        z = oracle.partial_dot_listing1_f32(x, y, use_fma=fma)
        ref = (x.astype(np.int64) * y.astype(np.int64)).reshape(9, 128).sum(axis=1)
        assert np.array_equal(z.astype(np.int64), ref)


def test_listing1_fp32_close_to_fp64():
    n = 128 * 64
    x = rand_f32(0, (n,))
    y = rand_f32(1, (n,))
    z32 = oracle.partial_dot_listing1_f32(x, y)
    z64, mag = oracle.partial_dot(x, y)
    # 7 rounding steps per result (2 in the pair, 6 tree levels) at 2^-24 each
    assert np.all(np.abs(z32 - z64) <= 8 * 2.0 ** -24 * mag + 1e-30)


# ---------------------------------------------------------------------------
# acceptance test helper
# ---------------------------------------------------------------------------

def test_within_tol_semantics():
    ok, margin = oracle.within_tol([1.0 + 5e-6], [1.0], [1.0])
    assert ok and 0.4 < margin < 0.6
    ok, _ = oracle.within_tol([1.0 + 2e-5], [1.0], [1.0])
    assert not ok
    ok, _ = oracle.within_tol([float("nan")], [1.0], [1.0])
    assert not ok


# ---------------------------------------------------------------------------
# the whole dot in Listing 1's structure (reading R26)
# ---------------------------------------------------------------------------

@pytest.mark.parametrize("use_fma", [True, False])
def test_dot_listing1_multistage_hand_derived(use_fma):
    case = golden("listing1_fp32_order.json")["multistage_cases"][0]
    x = np.zeros(case["n"], np.float32)
    for k, v in case["x"].items():
        x[int(k)] = v
    y = np.full(case["n"], case["y_all"], np.float32)
    assert oracle.dot_listing1_f32(x, y, use_fma) == case["expected"]


@pytest.mark.parametrize("n", [1, 5, 127, 128, 129, 128 * 128, 128 * 128 + 7, 3 * 128 * 128 * 2 + 1])
def test_dot_listing1_integer_exact(n):
    x = synth.small_ints(71, n, 3)
    y = synth.small_ints(72, n, 3)
    ref = int((x.astype(np.int64) * y.astype(np.int64)).sum())
    for fma in (True, False):
        assert oracle.dot_listing1_f32(x, y, fma) == float(ref)


def test_dot_listing1_single_group_is_partial_dot():
    x = rand_f32(0, (128,))
    y = rand_f32(1, (128,))
    for fma in (True, False):
        assert oracle.dot_listing1_f32(x, y, fma) == float(oracle.partial_dot_listing1_f32(x, y, fma)[0])
    # n < 128: the zero-padded single chunk
    xs, ys = x[:77], y[:77]
    xp, yp = np.zeros(128, np.float32), np.zeros(128, np.float32)
    xp[:77], yp[:77] = xs, ys
    assert oracle.dot_listing1_f32(xs, ys) == float(oracle.partial_dot_listing1_f32(xp, yp)[0])


def test_dot_listing1_close_to_fp64_and_empty():
    assert oracle.dot_listing1_f32(np.zeros(0, np.float32), np.zeros(0, np.float32)) == 0.0
    n = 1 << 20
    x = rand_f32(0, (n,))
    y = rand_f32(1, (n,))
    s64, mag = oracle.dot(x, y)
    # depth: 2 pair folds + 6 tree levels per stage, 3 stages at 2^20
    assert abs(oracle.dot_listing1_f32(x, y) - s64) <= 24 * 2.0 ** -24 * mag


# ---------------------------------------------------------------------------
# BLAS SGEMV (NEXT-4; CLBlast contract for Table 1's GEMV)
# ---------------------------------------------------------------------------

def _stored(Amat, layout, lda):
    """Store the logical m x n matrix in a padded buffer (padding = NaN, never read)."""
    m, n = Amat.shape
    if layout == 0:
        buf = np.full((m, lda), np.nan, np.float32)
        buf[:, :n] = Amat
    else:
        buf = np.full((n, lda), np.nan, np.float32)
        buf[:, :m] = Amat.T
    return buf


@pytest.mark.parametrize("layout", [0, 1])
@pytest.mark.parametrize("trans", [0, 1])
@pytest.mark.parametrize("alpha,beta", [(1.0, 0.0), (-0.5, 2.0), (1.5, 1.2)])
def test_sgemv_bruteforce_fraction(layout, trans, alpha, beta):
    m, n = 5, 7
    Am = rand_f32(2, (m, n))
    lda = (n if layout == 0 else m) + 3
    buf = _stored(Am, layout, lda)
    x = rand_f32(0, (m if trans else n,))
    yin = rand_f32(9, (n if trans else m,))
    y, mag = oracle.sgemv(layout, trans, m, n, alpha, buf, lda, x, beta, yin)
    opA = Am.T if trans else Am
    a32, b32 = F(np.float32(alpha)), F(np.float32(beta))
    exact = [a32 * s + (b32 * F(yv) if beta != 0 else 0) for s, yv in zip(exact_matvec(opA, x), yin)]
    assert np.all(np.isfinite(y))  # the NaN padding is never read
    assert_close_exact(y, exact, opA.shape[1] + 2, mag)
    # mag = |alpha| sum_k |op(A)_ok x_k| (+ |beta y_o| when beta != 0), exactly the sum of |terms|
    exact_mag = [abs(a32) * s + (abs(b32 * F(yv)) if beta != 0 else 0)
                 for s, yv in zip(exact_abs_matvec(opA, x), yin)]
    assert_close_exact(mag, exact_mag, opA.shape[1] + 2, mag)


def test_sgemv_reduces_to_gemv_and_ignores_y_when_beta_zero():
    m, n = 6, 9
    Am = rand_f32(2, (m, n))
    x = rand_f32(0, (n,))
    y, _ = oracle.sgemv(0, 0, m, n, 1.0, Am, n, x, 0.0, np.full(m, np.nan, np.float32))
    g, _ = oracle.gemv(Am, x)
    assert np.array_equal(y, g)
    # column-major storage of A^T read as row-major A: same result
    yt, _ = oracle.sgemv(1, 1, n, m, 1.0, Am, n, x, 0.0)
    assert np.array_equal(yt, g)
