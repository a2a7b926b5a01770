"""Seeded synthetic inputs shared by the oracle side and the CUDA side.

This module holds NO arithmetic of the method (no products, no sums of the
operands).  It only turns (seed, element index) into an fp32 value with a
counter-based hash, so any rank / device / process can regenerate any slice of
any operand without materialising the rest.  It exists because the paper's
data sets are not shipped ("Provided with the corresponding benchmarks",
PAPER.md L1316, App. A) and every workload here is synthetic.

Two implementations of the SAME generator are provided and tested bitwise
equal on CPU (tests/test_synth.py):

* ``numpy_*``  — uint32 arithmetic in numpy (host: oracle inputs, CPU bench leg)
* ``torch_*``  — int64 arithmetic with explicit 32-bit masking, usable on any
  torch device (GPU inputs are generated in HBM, outside every timed region).

Generator (per element with flat row-major index ``i`` and seed ``s``)::

    k = lowbias32(s ^ lowbias32(hi32(i) + 0x68E31DA4))
    h = lowbias32(lo32(i) ^ k)
    u = h >> 8                      # 24 uniform bits
    U[-1,1):  u * 2^-23 - 1         # exactly representable in fp32
    U[0,1):   u * 2^-24

``lowbias32`` is the public-domain 32-bit integer finaliser
``x ^= x>>16; x *= 0x7feb352d; x ^= x>>15; x *= 0x846ca68b; x ^= x>>16``.

Seeds follow SURVEY.md §8(d): x <- 0, y <- 1, A <- 2, B <- 3.
"""
from __future__ import annotations

import numpy as np

SEED_X, SEED_Y, SEED_A, SEED_B = 0, 1, 2, 3

_C1 = 0x7FEB352D
_C2 = 0x846CA68B
_HI_SALT = 0x68E31DA4
_M32 = 0xFFFFFFFF

# --------------------------------------------------------------------------
# numpy implementation (uint32 wraps natively)
# --------------------------------------------------------------------------


def _np_lowbias32(x: np.ndarray) -> np.ndarray:
    x = x.astype(np.uint32, copy=True)
    x ^= x >> np.uint32(16)
    x *= np.uint32(_C1)
    x ^= x >> np.uint32(15)
    x *= np.uint32(_C2)
    x ^= x >> np.uint32(16)
    return x


def numpy_bits(seed: int, start: int, count: int) -> np.ndarray:
    """24-bit uniform integers for flat indices [start, start+count)."""
    idx = np.arange(start, start + count, dtype=np.uint64)
    lo = (idx & np.uint64(_M32)).astype(np.uint32)
    hi = (idx >> np.uint64(32)).astype(np.uint32)
    with np.errstate(over="ignore"):
        k = _np_lowbias32(np.uint32(seed & _M32) ^ _np_lowbias32(hi + np.uint32(_HI_SALT)))
        h = _np_lowbias32(lo ^ k)
    return h >> np.uint32(8)


def numpy_uniform(seed: int, start: int, count: int, dist: str = "sym") -> np.ndarray:
    """fp32 values for flat indices [start, start+count).

    dist = "sym" -> U[-1,1) on a 2^-23 grid; "pos" -> U[0,1) on a 2^-24 grid.
    """
    u = numpy_bits(seed, start, count).astype(np.float64)
    if dist == "sym":
        v = u * 2.0 ** -23 - 1.0
    elif dist == "pos":
        v = u * 2.0 ** -24
    else:
        raise ValueError(f"unknown dist {dist!r}")
    return v.astype(np.float32)  # exact: at most 24 significant bits


_WIDE_SALT = 0x5BD1E995


def numpy_wide(seed: int, start: int, count: int, emin: int = -140, emax: int = 20) -> np.ndarray:
    """Wide-dynamic-range fp32 for flat indices [start, start+count): full 24-bit
    significands, binary exponents uniform in [emin, emax] (the default reaches
    into the subnormal range below 2^-126) and random signs.  Host side only;
    for the property tests (no value of the method's arithmetic is involved)."""
    mant = (numpy_bits(seed, start, count) >> np.uint32(1)).astype(np.float64)  # 23 fraction bits
    eb = numpy_bits(seed ^ _WIDE_SALT, start, count).astype(np.int64)  # exponent + sign bits
    e = emin + (eb >> 1) % (emax - emin + 1)
    sign = np.where(eb & 1, -1.0, 1.0)
    v = sign * (1.0 + mant * 2.0 ** -23) * np.exp2(e.astype(np.float64))
    return v.astype(np.float32)  # rounds the subnormal ones (deterministically)


def numpy_matrix_rows(seed: int, n_cols: int, r0: int, r1: int, dist: str = "sym") -> np.ndarray:
    """Rows [r0, r1) of the row-major matrix with ``n_cols`` columns."""
    return numpy_uniform(seed, r0 * n_cols, (r1 - r0) * n_cols, dist).reshape(r1 - r0, n_cols)


# --------------------------------------------------------------------------
# torch implementation (int64 lanes, explicit mod-2^32 multiply that never
# overflows int64: c = c_hi*2^16 + c_lo, x*c_lo < 2^48, (x*c_hi mod 2^16) << 16)
# --------------------------------------------------------------------------


def _t_mul32(x, c: int):
    c_lo, c_hi = c & 0xFFFF, c >> 16
    return (x * c_lo + (((x * c_hi) & 0xFFFF) << 16)) & _M32


def _t_lowbias32(x):
    x = x ^ (x >> 16)
    x = _t_mul32(x, _C1)
    x = x ^ (x >> 15)
    x = _t_mul32(x, _C2)
    x = x ^ (x >> 16)
    return x


def torch_uniform(seed: int, start: int, count: int, dist: str = "sym", device="cpu",
                  out=None, chunk: int = 1 << 26):
    """Same values as :func:`numpy_uniform`, produced by torch ops on ``device``.

    Generated in chunks so a 2^31-element operand needs only O(chunk) scratch.
    Writes into ``out`` (fp32, ``count`` elements) when given.
    """
    import torch

    if out is None:
        out = torch.empty(count, dtype=torch.float32, device=device)
    flat = out.view(-1)
    assert flat.numel() == count
    seed32 = seed & _M32
    for off in range(0, count, chunk):
        c = min(chunk, count - off)
        idx = torch.arange(start + off, start + off + c, dtype=torch.int64, device=flat.device)
        lo = idx & _M32
        hi = idx >> 32
        k = _t_lowbias32(seed32 ^ _t_lowbias32((hi + _HI_SALT) & _M32))
        h = _t_lowbias32(lo ^ k)
        u = (h >> 8).to(torch.float32)  # < 2^24: exact
        if dist == "sym":
            v = u * (2.0 ** -23) - 1.0  # exact in fp32 (see module doc)
        elif dist == "pos":
            v = u * (2.0 ** -24)
        else:
            raise ValueError(f"unknown dist {dist!r}")
        flat[off:off + c].copy_(v)
        del idx, lo, hi, k, h, u, v
    return out


def torch_matrix_rows(seed: int, n_cols: int, r0: int, r1: int, dist: str = "sym",
                      device="cpu", out=None):
    """Rows [r0, r1) of the seeded row-major matrix, as a (r1-r0, n_cols) tensor."""
    import torch

    if out is None:
        out = torch.empty((r1 - r0, n_cols), dtype=torch.float32, device=device)
    torch_uniform(seed, r0 * n_cols, (r1 - r0) * n_cols, dist, out=out)
    return out


# --------------------------------------------------------------------------
# structured inputs (closed-form cases of SURVEY.md §8(c)); numpy, host side
# --------------------------------------------------------------------------


def hadamard(n: int) -> np.ndarray:
    """Sylvester-Hadamard matrix H_ij = (-1)^popcount(i & j), n a power of two."""
    assert n > 0 and n & (n - 1) == 0
    i = np.arange(n, dtype=np.uint64)
    a = i[:, None] & i[None, :]
    # popcount parity by folding
    p = a.copy()
    for s in (32, 16, 8, 4, 2, 1):
        p ^= p >> np.uint64(s)
    return np.where((p & np.uint64(1)) == 0, 1.0, -1.0).astype(np.float32)


def small_ints(seed: int, count: int, lim: int) -> np.ndarray:
    """Integer-valued fp32 in [-lim, lim] from the same hash (exactness cases)."""
    b = numpy_bits(seed, 0, count).astype(np.int64)
    return ((b % (2 * lim + 1)) - lim).astype(np.float32)
