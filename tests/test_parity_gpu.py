"""GPU parity: the CUDA path (through the C ABI) against the fp64 oracle.

Acceptance (BASELINE.json north_star), elementwise:
    |y_gpu - y_ref| <= 1e-5 * mag + 1e-6,   mag = sum |terms| (from the oracle)
Integer-valued / structured inputs whose exact result is reached in fp32 in
ANY summation order are compared bitwise (SURVEY.md §8(c) pins).

Inputs come from synth (seeded, counter-based): small cases are generated on
the host and copied; BASELINE-size cases are generated in HBM by torch ops and
the oracle regenerates the sampled rows on the host from the same counters.
"""
import numpy as np
import pytest
import torch

import oracle
import synth
import paper_conf_cgo_steuwerrd17_b200 as lift

pytestmark = pytest.mark.gpu

ALPHA, BETA = 1.5, 1.2  # bench values (reading R9 / A9)


def dev_np(a, device):
    return torch.from_numpy(np.ascontiguousarray(a)).to(device)


def assert_tol(got, ref, mag, what=""):
    ok, margin = oracle.within_tol(got, ref, mag)
    assert ok, f"{what}: tolerance margin {margin:.3g} > 1"
    return margin


def rand(seed, shape, dist="sym"):
    return synth.numpy_uniform(seed, 0, int(np.prod(shape)), dist).reshape(shape)


# ===================================================================== dot
@pytest.mark.parametrize("n", [0, 1, 3, 4, 5, 127, 128, 129, 4097, 1 << 20, (1 << 20) + 3])
@pytest.mark.parametrize("dist", ["sym", "pos"])
def test_dot_parity(cuda_device, n, dist):
    x = rand(synth.SEED_X, (n,), dist)
    y = rand(synth.SEED_Y, (n,), dist)
    got = lift.lift_dot(dev_np(x, cuda_device), dev_np(y, cuda_device)).item()
    ref, mag = oracle.dot(x, y)
    assert_tol([got], [ref], [mag], f"dot n={n}")


@pytest.mark.parametrize("off", [1, 2, 3])
def test_dot_unaligned_scalar_path(cuda_device, off):
    n = 10007
    xb = dev_np(rand(0, (n + off,)), cuda_device)
    yb = dev_np(rand(1, (n + 4,)), cuda_device)
    x, y = xb[off:], yb[:n]
    got = lift.lift_dot(x, y).item()
    ref, mag = oracle.dot(x.cpu().numpy(), y.cpu().numpy())
    assert_tol([got], [ref], [mag], "dot unaligned")


def test_dot_exact_cases(cuda_device):
    for n in (1, 1000, 1 << 20, (1 << 24)):
        ones = torch.ones(n, device=cuda_device)
        assert lift.lift_dot(ones, ones).item() == float(n)
    alt = torch.ones(1 << 20, device=cuda_device)
    alt[1::2] = -1
    assert lift.lift_dot(alt, torch.ones_like(alt)).item() == 0.0
    assert lift.lift_dot(torch.zeros(0, device=cuda_device), torch.zeros(0, device=cuda_device)).item() == 0.0


def test_dot_deterministic_and_symmetric(cuda_device):
    n = (1 << 22) + 5
    x = synth.torch_uniform(0, 0, n, device=cuda_device)
    y = synth.torch_uniform(1, 0, n, device=cuda_device)
    a = lift.lift_dot(x, y).item()
    for _ in range(3):
        assert lift.lift_dot(x, y).item() == a
    assert lift.lift_dot(y, x).item() == a


def test_dot_ticket_rearms_across_many_calls(cuda_device):
    # the last-block ticket must return to zero every launch (else results go stale)
    n = 1 << 16
    ones = torch.ones(n, device=cuda_device)
    for k in range(1, 20):
        v = torch.full((n,), float(k), device=cuda_device)
        assert lift.lift_dot(v, ones).item() == float(k * n)


@pytest.mark.slow
def test_dot_full_size_2pow31(cuda_device):
    """configs[4]: 2^31-element dot (one GPU holds 16 GiB of x, y)."""
    n = 1 << 31
    x = synth.torch_uniform(synth.SEED_X, 0, n, device=cuda_device)
    y = synth.torch_uniform(synth.SEED_Y, 0, n, device=cuda_device)
    got = lift.lift_dot(x, y).item()
    del x, y
    torch.cuda.empty_cache()
    ref = 0.0
    mag = 0.0
    ch = 1 << 27
    for s in range(0, n, ch):  # reading A23: chunked fp64 folds agree to ~1e-12
        r, m = oracle.dot(synth.numpy_uniform(synth.SEED_X, s, ch), synth.numpy_uniform(synth.SEED_Y, s, ch))
        ref += r
        mag += m
    assert_tol([got], [ref], [mag], "dot 2^31")


# ===================================================================== GEMV
GEMV_SHAPES = [(1, 1), (7, 3), (5, 129), (3, 5000), (300, 1000), (1000, 4), (33, 4096), (257, 8192), (4096, 4096),
               (17, 32768),
               # extremes: x far beyond shared memory (16 MiB rows), ragged wide rows, very tall and skinny
               (2, 1 << 22), (3, (1 << 20) + 3), (1 << 20, 4), ((1 << 18) + 1, 3)]


@pytest.mark.parametrize("m,n", GEMV_SHAPES)
def test_gemv_parity(cuda_device, m, n):
    A = rand(synth.SEED_A, (m, n))
    x = rand(synth.SEED_X, (n,))
    got = lift.lift_gemv(dev_np(A, cuda_device), dev_np(x, cuda_device)).cpu().numpy()
    ref, mag = oracle.gemv(A, x)
    assert_tol(got, ref, mag, f"gemv {m}x{n}")


def test_gemv_positive_data_8192(cuda_device):
    m, n = 512, 8192
    A = rand(synth.SEED_A, (m, n), "pos")
    x = rand(synth.SEED_X, (n,), "pos")
    got = lift.lift_gemv(dev_np(A, cuda_device), dev_np(x, cuda_device)).cpu().numpy()
    ref, mag = oracle.gemv(A, x)
    assert_tol(got, ref, mag, "gemv positive")


def test_gemv_unaligned_and_ragged(cuda_device):
    m, n = 37, 1001
    buf = dev_np(rand(2, (m * n + 3,)), cuda_device)
    A = buf[3:].view(m, n)  # 12-byte offset: scalar path
    x = dev_np(rand(0, (n,)), cuda_device)
    got = lift.lift_gemv(A, x).cpu().numpy()
    ref, mag = oracle.gemv(A.cpu().numpy(), x.cpu().numpy())
    assert_tol(got, ref, mag, "gemv unaligned")


def test_gemv_empty(cuda_device):
    A = torch.zeros(5, 0, device=cuda_device)
    y = lift.lift_gemv(A, torch.zeros(0, device=cuda_device))
    assert torch.equal(y, torch.zeros(5, device=cuda_device))
    y = lift.lift_gemv(torch.zeros(0, 7, device=cuda_device), torch.zeros(7, device=cuda_device))
    assert y.numel() == 0


@pytest.mark.parametrize("n", [4096, 8192, 32768])
def test_gemv_exact_structured(cuda_device, n):
    m = 64
    ones = torch.ones(m, n, device=cuda_device)
    assert torch.equal(lift.lift_gemv(ones, torch.ones(n, device=cuda_device)), torch.full((m,), float(n), device=cuda_device))
    H = dev_np(synth.hadamard(256), cuda_device)
    for k in (0, 5, 255):
        e = torch.zeros(256, device=cuda_device)
        e[k] = 1
        assert torch.equal(lift.lift_gemv(H, e), H[:, k].contiguous())
    I = torch.eye(512, device=cuda_device)
    x = dev_np(rand(0, (512,)), cuda_device)
    assert torch.equal(lift.lift_gemv(I, x), x)


def test_gemv_config_invariant_and_shard_bitwise(cuda_device):
    """Canonical per-row order: every launch configuration and every row
    shard gives the same bits (what makes g-GPU == 1-GPU bitwise)."""
    m, n = 1000, 4096
    A = synth.torch_matrix_rows(synth.SEED_A, n, 0, m, device=cuda_device)
    x = synth.torch_uniform(synth.SEED_X, 0, n, device=cuda_device)
    base = lift.lift_gemv(A, x)
    for wpr, rg in ((8, 1), (8, 2), (4, 2), (4, 4), (2, 4), (2, 8), (1, 8)):
        for xs in (0, 1):
            for lb in (4, 8):
                got = lift.lift_gemv_tuned(A, x, wpr=wpr, rg=rg, xsmem=xs, lb=lb)
                assert torch.equal(got, base), (wpr, rg, xs, lb)
    got = lift.lift_gemv_tuned(A, x, blocks=3)
    assert torch.equal(got, base)
    for r0, r1 in ((0, 1), (0, 500), (500, 1000), (123, 877)):
        assert torch.equal(lift.lift_gemv(A[r0:r1], x), base[r0:r1])


def test_gemv_nan_propagates(cuda_device):
    m, n = 16, 256
    A = dev_np(rand(2, (m, n)), cuda_device)
    x = dev_np(rand(0, (n,)), cuda_device)
    x[17] = float("nan")
    assert torch.isnan(lift.lift_gemv(A, x)).all()


def test_nan_propagates_every_op(cuda_device):
    """Reading A14: IEEE propagation, no special-casing — a NaN
    input element reaches every output that depends on it, in every op and
    algorithm; outputs that do not depend on it stay finite."""
    m, n = 300, 1024
    A = dev_np(rand(2, (m, n)), cuda_device)
    B = dev_np(rand(3, (m, n)), cuda_device)
    x = dev_np(rand(0, (n,)), cuda_device)
    xn = x.clone()
    xn[517] = float("nan")
    assert torch.isnan(lift.lift_dot(xn, x)).item()
    assert torch.isnan(lift.lift_gesummv(1.5, A, 1.2, B, xn)).all()
    for algo in ("fused", "twopass"):
        assert torch.isnan(lift.lift_atax(A, xn, algo=algo)).all()  # t is all NaN, so is every y_j
    # a NaN in one row of A: only that row of A x, but (through t) every y_j of ATAX
    An = A.clone()
    An[123, 45] = float("nan")
    y = lift.lift_gemv(An, x)
    assert torch.isnan(y[123]) and torch.isfinite(torch.cat([y[:123], y[124:]])).all()
    for algo in ("fused", "twopass"):
        assert torch.isnan(lift.lift_atax(An, x, algo=algo)).all()


def test_gemv_nondefault_stream_and_graph(cuda_device):
    m, n = 2048, 4096
    A = synth.torch_matrix_rows(synth.SEED_A, n, 0, m, device=cuda_device)
    x = synth.torch_uniform(synth.SEED_X, 0, n, device=cuda_device)
    ref = lift.lift_gemv(A, x)
    s = torch.cuda.Stream()
    with torch.cuda.stream(s):
        y = torch.empty(m, device=cuda_device)
        lift.lift_gemv(A, x, out=y)
    s.synchronize()
    assert torch.equal(y, ref)
    g = torch.cuda.CUDAGraph()
    y2 = torch.empty(m, device=cuda_device)
    with torch.cuda.graph(g):
        lift.lift_gemv(A, x, out=y2)
    y2.zero_()
    g.replay()
    torch.cuda.synchronize()
    assert torch.equal(y2, ref)


def test_workspace_per_graph_capture(cuda_device):
    """Workspaces with counters (dot ticket, ATAX grid barrier) first made
    inside a graph capture are zeroed only when that graph replays: each
    capture gets its own, and each graph alone replays correctly."""
    from paper_conf_cgo_steuwerrd17_b200 import _ws_cache
    n = 1 << 20
    x = synth.torch_uniform(synth.SEED_X, 0, n, device=cuda_device)
    y = synth.torch_uniform(synth.SEED_Y, 0, n, device=cuda_device)
    A = synth.torch_matrix_rows(synth.SEED_A, 1024, 0, 700, device=cuda_device)
    xa = synth.torch_uniform(synth.SEED_X, 0, 1024, device=cuda_device)
    want_d, want_a = lift.lift_dot(x, y).clone(), lift.lift_atax(A, xa).clone()
    before = {k for k in _ws_cache if k[3] != 0}
    graphs, outs = [], []
    for _ in range(2):
        g = torch.cuda.CUDAGraph()
        d = torch.empty((), device=cuda_device)
        a = torch.empty(1024, device=cuda_device)
        with torch.cuda.graph(g):
            lift.lift_dot(x, y, out=d)
            lift.lift_atax(A, xa, out=a)
        graphs.append(g)
        outs.append((d, a))
    new = {k for k in _ws_cache if k[3] != 0} - before
    assert len({k[3] for k in new}) == 2 and {k[0] for k in new} == {"dot", "atax"}
    for g, (d, a) in reversed(list(zip(graphs, outs))):  # the second graph first, alone
        d.zero_()
        a.zero_()
        for _ in range(3):
            g.replay()
        torch.cuda.synchronize()
        assert torch.equal(d, want_d) and torch.equal(a, want_a)
    assert torch.equal(lift.lift_dot(x, y), want_d)  # the eager workspace is untouched


@pytest.mark.slow
def test_gemv_full_size_65536x32768_sampled(cuda_device):
    """configs[4] large GEMV (8 GiB A) in the bench's launch configuration;
    sampled rows checked against the oracle regenerated on the host."""
    m, n = 65536, 32768
    A = synth.torch_matrix_rows(synth.SEED_A, n, 0, m, device=cuda_device)
    x = synth.torch_uniform(synth.SEED_X, 0, n, device=cuda_device)
    y = lift.lift_gemv(A, x).cpu().numpy()
    rows = np.unique(np.concatenate([[0, 1, m - 1, m // 2], np.random.RandomState(7).randint(0, m, 60)]))
    xs = synth.numpy_uniform(synth.SEED_X, 0, n)
    As = np.stack([synth.numpy_matrix_rows(synth.SEED_A, n, r, r + 1)[0] for r in rows])
    ref, mag = oracle.gemv(As, xs)
    assert_tol(y[rows], ref, mag, "gemv 65536x32768 sampled")


# ===================================================================== GESUMMV
@pytest.mark.parametrize("m,n", [(1, 1), (9, 7), (100, 1000), (64, 4096), (1024, 8192), (3, 32768)])
@pytest.mark.parametrize("ab", [(ALPHA, BETA), (-0.75, 3.0), (0.0, 1.0), (1.0, 0.0), (-1.0, -1.0)])
def test_gesummv_parity(cuda_device, m, n, ab):
    al, be = ab
    A = rand(synth.SEED_A, (m, n))
    B = rand(synth.SEED_B, (m, n))
    x = rand(synth.SEED_X, (n,))
    got = lift.lift_gesummv(al, dev_np(A, cuda_device), be, dev_np(B, cuda_device), dev_np(x, cuda_device))
    ref, mag = oracle.gesummv(al, A, be, B, x)
    assert_tol(got.cpu().numpy(), ref, mag, f"gesummv {m}x{n} {ab}")


def test_gesummv_full_size_8192(cuda_device):
    """configs[2] at one GPU, every row."""
    m = n = 8192
    A = synth.torch_matrix_rows(synth.SEED_A, n, 0, m, device=cuda_device)
    B = synth.torch_matrix_rows(synth.SEED_B, n, 0, m, device=cuda_device)
    x = synth.torch_uniform(synth.SEED_X, 0, n, device=cuda_device)
    got = lift.lift_gesummv(ALPHA, A, BETA, B, x).cpu().numpy()
    ref, mag = oracle.gesummv(ALPHA, A.cpu().numpy(), BETA, B.cpu().numpy(), x.cpu().numpy())
    assert_tol(got, ref, mag, "gesummv 8192")


def test_gesummv_reductions_bitwise(cuda_device):
    m, n = 300, 4096
    A = synth.torch_matrix_rows(synth.SEED_A, n, 0, m, device=cuda_device)
    B = synth.torch_matrix_rows(synth.SEED_B, n, 0, m, device=cuda_device)
    x = synth.torch_uniform(synth.SEED_X, 0, n, device=cuda_device)
    g = lift.lift_gemv(A, x)
    # same canonical row order in both kernels: beta = 0 gives alpha * gemv exactly
    assert torch.equal(lift.lift_gesummv(ALPHA, A, 0.0, B, x), ALPHA * g)
    assert torch.equal(lift.lift_gesummv(1.0, A, 0.0, B, x), g)
    assert torch.equal(lift.lift_gesummv(0.0, B, 1.0, A, x), g)
    # ones: (alpha + beta) * n exactly
    ones = torch.ones(8, n, device=cuda_device)
    got = lift.lift_gesummv(1.5, ones, 1.25, ones, torch.ones(n, device=cuda_device))
    assert torch.equal(got, torch.full((8,), 2.75 * n, device=cuda_device))
    # sharded rows bitwise
    full = lift.lift_gesummv(ALPHA, A, BETA, B, x)
    assert torch.equal(lift.lift_gesummv(ALPHA, A[100:200], BETA, B[100:200], x), full[100:200])


# ===================================================================== ATAX
ATAX_SHAPES = [(1, 1), (5, 3), (3, 7), (64, 32), (1000, 300), (300, 1001), (4096, 4096), (2000, 16384), (100, 20000)]


def cluster_of(n: int) -> int:
    """Cluster size the single-pass ATAX uses for wide rows: the smallest C whose
    column slices are whole float4 columns, at most 4096 float4."""
    return next(c for c in (2, 4, 8, 16) if n % (4 * c) == 0 and n // c // 4 <= 4096)


def fused_supported(n: int) -> bool:
    """Shapes the single-pass ATAX accepts (16-B aligned operands): n % 4 == 0 and
    either n <= 16384 (one block per row) or a cluster of C in {2, 4, 8, 16}
    blocks whose column slices are whole float4 columns, at most 2048 float4."""
    if n % 4:
        return False
    if n <= 16384:
        return True
    for c in (2, 4, 8, 16):
        if n % (4 * c):
            return False
        if n // c // 4 <= 4096:
            return True
    return False


@pytest.mark.parametrize("m,n", ATAX_SHAPES)
@pytest.mark.parametrize("algo", ["auto", "fused", "twopass"])
def test_atax_parity(cuda_device, m, n, algo):
    A = rand(synth.SEED_A, (m, n))
    x = rand(synth.SEED_X, (n,))
    Ad, xd = dev_np(A, cuda_device), dev_np(x, cuda_device)
    if algo == "fused" and not fused_supported(n):
        with pytest.raises(lift.LiftError):
            lift.lift_atax(Ad, xd, algo=algo)
        return
    got = lift.lift_atax(Ad, xd, algo=algo).cpu().numpy()
    ref, mag = oracle.atax(A, x)
    assert_tol(got, ref, mag, f"atax {m}x{n} {algo}")


def test_atax_fused_tuning(cuda_device):
    """lift_atax_fused_tuned: the ring depth changes only the speed (bitwise
    equal results, at every width — up to 16384 the single-block kernel, beyond
    it the cluster kernel); the row assignment (banded / cyclic) changes which
    rows each block's partial sums, so both are checked against the oracle, and
    the automatic setting is the cyclic one bitwise; unsupported settings are
    rejected."""
    for m, n in ((1000, 4096), (777, 8192), (600, 12288), (300, 16384), (5000, 512), (300, 32768)):
        A = synth.torch_matrix_rows(synth.SEED_A, n, 0, m, device=cuda_device)
        x = synth.torch_uniform(synth.SEED_X, 0, n, device=cuda_device)
        ref, mag = oracle.atax(A.cpu().numpy(), x.cpu().numpy())
        auto = lift.lift_atax(A, x, algo="fused")
        for cyc in ((0, 1) if n <= 16384 else (1,)):
            base = lift.lift_atax_fused_tuned(A, x, cyclic=cyc)
            assert_tol(base.cpu().numpy(), ref, mag, f"atax tuned {m}x{n} cyc {cyc}")
            if cyc == 1:
                assert torch.equal(base, auto), (m, n)
            for nst in (2, 3, 5):
                try:
                    got = lift.lift_atax_fused_tuned(A, x, nst=nst, cyclic=cyc)
                except lift.LiftError:  # ring does not fit the shared-memory budget
                    assert n > 8192 and nst >= 3, (m, n, nst)  # 64 KiB rows + x in smem: 2 stages max
                    continue
                assert torch.equal(got, base), (m, n, cyc, nst)
        bads = [dict(nst=1), dict(nst=17), dict(cyclic=2)] + ([dict(cyclic=0)] if n > 16384 else [])
        for bad in bads:
            with pytest.raises(lift.LiftError):
                lift.lift_atax_fused_tuned(A, x, **bad)


WIDE_SHAPES = [(1, 16416), (7, 16392), (3, 20000), (300, 32768), (1001, 24576), (64, 65536), (777, 16416), (2048, 32768),
               (9, 16400), (5, 131072), (130, 49152)]


@pytest.mark.parametrize("m,n", WIDE_SHAPES)
def test_atax_fused_wide(cuda_device, m, n):
    """Single-pass ATAX for rows wider than one block can ring-buffer
    (n > 16384): the columns split over a thread-block cluster, row dots
    pushed as warp sums into every block's shared memory by asynchronous
    remote stores.  Oracle tolerance, bitwise repeatable, chosen by
    algo="auto" where it is the faster algorithm (n = 32768 here), and within
    tolerance of the two-pass algorithm."""
    assert fused_supported(n)
    A = synth.torch_matrix_rows(synth.SEED_A, n, 0, m, device=cuda_device)
    x = synth.torch_uniform(synth.SEED_X, 0, n, device=cuda_device)
    ref, mag = oracle.atax(A.cpu().numpy(), x.cpu().numpy())
    got = lift.lift_atax(A, x, algo="fused")
    assert_tol(got.cpu().numpy(), ref, mag, f"atax wide {m}x{n}")
    for _ in range(2):
        assert torch.equal(lift.lift_atax(A, x, algo="fused"), got)
    auto = lift.lift_atax(A, x)  # the single pass where it beats the two-pass algorithm
    assert_tol(auto.cpu().numpy(), ref, mag, f"atax auto {m}x{n}")
    assert torch.equal(auto, got)  # auto takes the single pass for every supported wide row
    assert_tol(lift.lift_atax(A, x, algo="twopass").cpu().numpy(), ref, mag, f"atax twopass {m}x{n}")


def test_atax_fused_grid(cuda_device):
    """lift_atax_fused_grid reports the single pass's launch shape: one block per SM
    up to 16384 columns, whole clusters of the wide kernel beyond (at most one
    block per SM), and the wide kernel's cluster is the one its slices need."""
    sms = torch.cuda.get_device_properties(cuda_device).multi_processor_count
    assert lift.lift_atax_fused_grid(8192, 8192) == (min(sms, 256), 1)
    assert lift.lift_atax_fused_grid(5, 4096) == (5, 1)
    for n in (20000, 32768, 65536, 131072):
        blocks, c = lift.lift_atax_fused_grid(8192, n)
        assert c == cluster_of(n) and blocks % c == 0 and 0 < blocks <= sms, (n, blocks, c)
    c = cluster_of(32768)
    assert lift.lift_atax_fused_grid(3, 32768) == (3 * c, c)  # one cluster per row


def test_atax_fused_wide_rejects(cuda_device):
    """Wide rows whose cluster slices would not be whole float4 columns stay on
    the two-pass algorithm (auto) and are refused by algo="fused"."""
    for n in (16388, 20004, 32772):
        assert not fused_supported(n)
        A = synth.torch_matrix_rows(synth.SEED_A, n, 0, 5, device=cuda_device)
        x = synth.torch_uniform(synth.SEED_X, 0, n, device=cuda_device)
        with pytest.raises(lift.LiftError):
            lift.lift_atax(A, x, algo="fused")
        ref, mag = oracle.atax(A.cpu().numpy(), x.cpu().numpy())
        assert_tol(lift.lift_atax(A, x).cpu().numpy(), ref, mag, f"atax auto {n}")


@pytest.mark.parametrize("algo", ["fused", "twopass"])
def test_atax_full_size_8192(cuda_device, algo):
    """configs[3] at one GPU, every output."""
    m = n = 8192
    A = synth.torch_matrix_rows(synth.SEED_A, n, 0, m, device=cuda_device)
    x = synth.torch_uniform(synth.SEED_X, 0, n, device=cuda_device)
    got = lift.lift_atax(A, x, algo=algo).cpu().numpy()
    ref, mag = oracle.atax(A.cpu().numpy(), x.cpu().numpy())
    assert_tol(got, ref, mag, f"atax 8192 {algo}")


@pytest.mark.parametrize("algo", ["fused", "twopass"])
def test_atax_exact_structured(cuda_device, algo):
    n = 4096
    H = dev_np(synth.hadamard(n), cuda_device)
    for k in (0, 77, n - 1):
        e = torch.zeros(n, device=cuda_device)
        e[k] = 1
        want = torch.zeros(n, device=cuda_device)
        want[k] = n
        assert torch.equal(lift.lift_atax(H, e, algo=algo), want)  # H^T H = n I
    x = dev_np(rand(0, (1024,)), cuda_device)
    I = torch.eye(1024, device=cuda_device)
    assert torch.equal(lift.lift_atax(I, x, algo=algo), x)
    perm = torch.randperm(1024, generator=torch.Generator().manual_seed(0))
    P = I[perm].contiguous()
    assert torch.equal(lift.lift_atax(P, x, algo=algo), x)


def test_atax_empty(cuda_device):
    y = lift.lift_atax(torch.zeros(0, 9, device=cuda_device), torch.ones(9, device=cuda_device))
    assert torch.equal(y, torch.zeros(9, device=cuda_device))


def test_atax_deterministic(cuda_device):
    m, n = 3000, 4096
    A = synth.torch_matrix_rows(synth.SEED_A, n, 0, m, device=cuda_device)
    x = synth.torch_uniform(synth.SEED_X, 0, n, device=cuda_device)
    for algo in ("fused", "twopass"):
        a = lift.lift_atax(A, x, algo=algo)
        for _ in range(3):
            assert torch.equal(lift.lift_atax(A, x, algo=algo), a)


@pytest.mark.parametrize("m,n", [(3000, 4096), (8192, 8192), (700, 16384), (513, 96)])
def test_partial_rows_discard_is_invisible(cuda_device, m, n):
    """The partial-sum rows are dropped from L2 after their last read
    (discard.global.L2) only when each row is whole 128-byte lines; a
    workspace offset by 16 bytes turns that off.  Results must be bitwise the
    same either way, and across repeated calls that rewrite discarded lines
    (fused ATAX; the two-pass ATAX and the transposed SGEMV, whose column sums
    do not discard, are checked the same way)."""
    L = lift.lib()
    A = synth.torch_matrix_rows(synth.SEED_A, n, 0, m, device=cuda_device)
    x = synth.torch_uniform(synth.SEED_X, 0, n, device=cuda_device)
    xt = synth.torch_uniform(synth.SEED_Y, 0, m, device=cuda_device)
    stream = torch.cuda.current_stream(cuda_device).cuda_stream

    def ws_pair(nbytes):
        a = torch.zeros(nbytes + 512, dtype=torch.uint8, device=cuda_device)
        b = torch.zeros(nbytes + 512, dtype=torch.uint8, device=cuda_device)
        return a, b[16:]  # 256-byte aligned base (discard on) / 16-byte offset (off)

    for algo in (lift.LIFT_ATAX_FUSED, lift.LIFT_ATAX_TWOPASS):
        nb = L.lift_atax_workspace_bytes(m, n)
        outs = []
        for ws in ws_pair(nb):
            for _ in range(3):
                y = torch.empty(n, device=cuda_device)
                lift.check(L.lift_atax_algo_run(algo, m, n, A.data_ptr(), x.data_ptr(), y.data_ptr(),
                                                ws.data_ptr(), nb, stream))
                outs.append(y)
        assert all(torch.equal(o, outs[0]) for o in outs), algo
    nb = L.lift_sgemv_workspace_bytes(0, 1, m, n)
    outs = []
    for ws in ws_pair(nb):
        for _ in range(3):
            y = torch.full((n,), 0.25, device=cuda_device)
            lift.check(L.lift_sgemv(0, 1, m, n, 1.5, A.data_ptr(), n, xt.data_ptr(), 0.5, y.data_ptr(),
                                    ws.data_ptr(), nb, stream))
            outs.append(y)
    assert all(torch.equal(o, outs[0]) for o in outs)
    if m * n <= 1 << 24:
        ref, mag = oracle.atax(A.cpu().numpy(), x.cpu().numpy())
        assert_tol(lift.lift_atax(A, x, algo="fused").cpu().numpy(), ref, mag, "atax after discards")


def test_atax_unaligned(cuda_device):
    m, n = 50, 301
    buf = dev_np(rand(2, (m * n + 1,)), cuda_device)
    A = buf[1:].view(m, n)
    x = dev_np(rand(0, (n,)), cuda_device)
    got = lift.lift_atax(A, x).cpu().numpy()
    ref, mag = oracle.atax(A.cpu().numpy(), x.cpu().numpy())
    assert_tol(got, ref, mag, "atax unaligned")


# ===================================================================== Listing 1, bit for bit (NEXT-3)
@pytest.mark.parametrize("n", [128, 256, 128 * 37, 1 << 16, (1 << 20) + 77])
@pytest.mark.parametrize("contract", [True, False])
def test_partial_dot_listing1_bitwise(cuda_device, n, contract):
    x = rand(synth.SEED_X, (n,))
    y = rand(synth.SEED_Y, (n,))
    got = lift.lift_partial_dot(dev_np(x, cuda_device), dev_np(y, cuda_device), contract=contract).cpu().numpy()
    ref = oracle.partial_dot_listing1_f32(x, y, use_fma=contract)
    assert got.shape == ref.shape
    assert np.array_equal(got.view(np.uint32), ref.view(np.uint32))
    # and the plain-definition tolerance against fp64
    z64, mag = oracle.partial_dot(x, y)
    assert_tol(got, z64, mag, "partialDot vs fp64")


@pytest.mark.parametrize("n", [0, 1, 127, 128, 129, 128 * 128, 128 * 128 + 1, (1 << 22) + 3, 3 * (1 << 21)])
@pytest.mark.parametrize("contract", [True, False])
def test_dot_listing1_bitwise(cuda_device, n, contract):
    x = rand(synth.SEED_X, (n,))
    y = rand(synth.SEED_Y, (n,))
    got = lift.lift_dot_listing1(dev_np(x, cuda_device), dev_np(y, cuda_device), contract=contract).item()
    ref = oracle.dot_listing1_f32(x, y, use_fma=contract)
    assert np.float32(got).view(np.uint32) == np.float32(ref).view(np.uint32), (got, ref)
    s64, mag = oracle.dot(x, y)
    assert_tol([got], [s64], [mag], "dot_listing1 vs fp64")


def test_partial_dot_listing1_golden_cases(cuda_device):
    from conftest import golden

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
        for contract, key in ((True, "expected_fma"), (False, "expected_nofma")):
            z = lift.lift_partial_dot(dev_np(x, cuda_device), dev_np(y, cuda_device), contract=contract)
            assert float(z.item()) == case[key], (case["name"], contract)
    mc = g["multistage_cases"][0]
    x = np.zeros(mc["n"], np.float32)
    for k, v in mc["x"].items():
        x[int(k)] = v
    y = np.full(mc["n"], mc["y_all"], np.float32)
    assert lift.lift_dot_listing1(dev_np(x, cuda_device), dev_np(y, cuda_device)).item() == mc["expected"]


def test_partial_dot_unaligned(cuda_device):
    n = 128 * 50 + 3
    xb = dev_np(rand(0, (n + 1,)), cuda_device)
    yb = dev_np(rand(1, (n + 2,)), cuda_device)
    x, y = xb[1:], yb[2:]
    got = lift.lift_partial_dot(x, y).cpu().numpy()
    ref = oracle.partial_dot_listing1_f32(x.cpu().numpy(), y.cpu().numpy())
    assert np.array_equal(got.view(np.uint32), ref.view(np.uint32))


# ===================================================================== BLAS SGEMV (NEXT-4)
@pytest.mark.parametrize("layout", ["row", "col"])
@pytest.mark.parametrize("trans", [False, True])
@pytest.mark.parametrize("m,n,pad", [(300, 1000, 0), (333, 517, 3), (4096, 4096, 4), (7, 3, 1), (0, 5, 0), (5, 0, 0)])
@pytest.mark.parametrize("alpha,beta", [(1.0, 0.0), (1.5, 1.2), (-2.0, 0.5)])
def test_sgemv_parity(cuda_device, layout, trans, m, n, pad, alpha, beta):
    lay = 0 if layout == "row" else 1
    rows, cols = (m, n) if lay == 0 else (n, m)
    lda = max(cols, 1) + pad
    buf = synth.numpy_uniform(synth.SEED_A, 0, rows * lda).reshape(rows, lda) if rows else np.zeros((0, lda), np.float32)
    x = rand(synth.SEED_X, (m if trans else n,))
    ylen = n if trans else m
    yin = rand(9, (ylen,))
    yd = dev_np(yin, cuda_device)
    if beta == 0.0:
        yd.fill_(float("nan"))  # must not be read
    lift.lift_sgemv(alpha, dev_np(buf, cuda_device), dev_np(x, cuda_device), beta, yd, trans=trans, layout=layout,
                    lda=lda, shape=(m, n))
    ref, mag = oracle.sgemv(lay, int(trans), m, n, alpha, buf, lda, x, beta, yin)
    assert_tol(yd.cpu().numpy(), ref, mag, f"sgemv {layout} trans={trans} {m}x{n}")


def test_sgemv_alpha1_beta0_is_gemv_bitwise(cuda_device):
    m, n = 777, 4096
    A = synth.torch_matrix_rows(synth.SEED_A, n, 0, m, device=cuda_device)
    x = synth.torch_uniform(synth.SEED_X, 0, n, device=cuda_device)
    assert torch.equal(lift.lift_sgemv(1.0, A, x), lift.lift_gemv(A, x))
    # y = 2*(Ax) - 1*y applied twice from y = Ax gives Ax exactly (power-of-two scalings)
    y = lift.lift_gemv(A, x)
    ref = y.clone()
    lift.lift_sgemv(2.0, A, x, -1.0, y)
    assert torch.equal(y, ref)


# ===================================================================== host-buffer entry points
@pytest.mark.parametrize("pinned", [True, False])
def test_host_entry_points_match_device_path(cuda_device, pinned):
    m, n = 1000, 4096
    A = synth.numpy_matrix_rows(synth.SEED_A, n, 0, m)
    B = synth.numpy_matrix_rows(synth.SEED_B, n, 0, m)
    x = synth.numpy_uniform(synth.SEED_X, 0, n)

    def host(a):
        t = torch.from_numpy(np.ascontiguousarray(a))
        return t.pin_memory() if pinned else t.clone()

    Ad, Bd, xd = dev_np(A, cuda_device), dev_np(B, cuda_device), dev_np(x, cuda_device)
    cases = {
        "gemv": (dict(A=host(A), x=host(x), out=host(np.zeros(m, np.float32))),
                 dict(A=torch.empty_like(Ad), x=torch.empty_like(xd), out=torch.empty(m, device=cuda_device)),
                 lift.lift_gemv(Ad, xd)),
        "gesummv": (dict(A=host(A), B=host(B), x=host(x), out=host(np.zeros(m, np.float32))),
                    dict(A=torch.empty_like(Ad), B=torch.empty_like(Bd), x=torch.empty_like(xd),
                         out=torch.empty(m, device=cuda_device)),
                    lift.lift_gesummv(1.5, Ad, 1.2, Bd, xd)),
        "atax": (dict(A=host(A), x=host(x), out=host(np.zeros(n, np.float32))),
                 dict(A=torch.empty_like(Ad), x=torch.empty_like(xd), out=torch.empty(n, device=cuda_device)),
                 lift.lift_atax(Ad, xd)),
        "dot": (dict(x=host(A.ravel()), y=host(B.ravel()), out=host(np.zeros((), np.float32))),
                dict(x=torch.empty(m * n, device=cuda_device), y=torch.empty(m * n, device=cuda_device),
                     out=torch.empty((), device=cuda_device)),
                lift.lift_dot(Ad.view(-1), Bd.view(-1))),
    }
    for op, (h, d, ref) in cases.items():
        lift.lift_host_call(op, h, d, alpha=1.5, beta=1.2)
        torch.cuda.synchronize()
        assert torch.equal(h["out"].reshape(-1), ref.cpu().reshape(-1)), op


# ===================================================================== binding extents
def test_binding_rejects_wrong_output_extents(cuda_device):
    """The C ABI takes bare pointers and cannot see a buffer's extent: the binding
    rejects an output (or tuned input) of the wrong length or device before any
    launch, so a short tensor is never written past its end."""
    m, n = 64, 256
    A = synth.torch_matrix_rows(synth.SEED_A, n, 0, m, device=cuda_device)
    x = synth.torch_uniform(synth.SEED_X, 0, n, device=cuda_device)
    short_m, short_n = torch.empty(m - 1, device=cuda_device), torch.empty(n - 4, device=cuda_device)
    bad = [
        lambda: lift.lift_gemv(A, x, out=short_m),
        lambda: lift.lift_gemv_tuned(A, x, out=short_m),
        lambda: lift.lift_gemv_tuned(A, x[:-4]),
        lambda: lift.lift_gesummv(1.0, A, 1.0, A, x, out=short_m),
        lambda: lift.lift_gesummv_tuned(1.0, A, 1.0, A[:-1], x),
        lambda: lift.lift_atax(A, x, out=short_n),
        lambda: lift.lift_atax_fused_tuned(A, x, out=short_n),
        lambda: lift.lift_dot(x, x, out=torch.empty(0, device=cuda_device)),
        lambda: lift.lift_dot_listing1(x, x, out=torch.empty(2, device=cuda_device)),
        lambda: lift.lift_partial_dot(x, x, out=torch.empty(1, device=cuda_device)),
        lambda: lift.lift_gemv(A, x, out=torch.empty(m)),  # host tensor
        lambda: lift.lift_sgemv(1.0, A[:10], x, shape=(m, n)),  # A shorter than the matrix
        lambda: lift.lift_host_call("gemv", dict(A=A.cpu(), x=x.cpu(), out=torch.empty(m)),
                                    dict(A=A, x=x, out=short_m)),
    ]
    for i, call in enumerate(bad):
        with pytest.raises((ValueError, TypeError)):
            call()
            pytest.fail(f"case {i} accepted")
    torch.cuda.synchronize()
    assert torch.equal(lift.lift_gemv_tuned(A, x), lift.lift_gemv(A, x))  # the checks pass valid calls
