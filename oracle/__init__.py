"""fp64 CPU oracle (ctypes wrapper over oracle/liboracle.so, built with gcc).

TEST INFRASTRUCTURE ONLY.  Only ``tests/``, ``__graft_entry__.smoke()`` and
``bench.py``'s ``cpu_baseline`` / ``--impl reference`` leg may import this
package.  It shares no code with the CUDA path and the product package never
imports it.  See oracle.h for the definitions and their PAPER.md citations.

All functions take numpy fp32 arrays and return fp64 results together with the
fp64 tolerance magnitude ``mag`` (sum of |terms|) for the acceptance test
``|y - y_ref| <= 1e-5 * mag + 1e-6`` (BASELINE.json north_star).
"""
from __future__ import annotations

import ctypes
import os
import subprocess

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_SO = os.path.join(_HERE, "liboracle.so")
_SRC = [os.path.join(_HERE, "oracle.c"), os.path.join(_HERE, "oracle.h")]

RTOL = 1e-5
ATOL = 1e-6


def build(force: bool = False) -> str:
    """Compile liboracle.so with gcc (no fast-math, no contraction)."""
    stale = not os.path.exists(_SO) or any(os.path.getmtime(s) > os.path.getmtime(_SO) for s in _SRC)
    if force or stale:
        cmd = ["gcc", "-O2", "-ffp-contract=off", "-fno-fast-math", "-fopenmp", "-fPIC", "-shared",
               "-Wall", "-Wextra", "-o", _SO + ".tmp", _SRC[0], "-lm"]
        subprocess.check_call(cmd, cwd=_HERE)
        os.replace(_SO + ".tmp", _SO)
    return _SO


_lib = None


def _load():
    global _lib
    if _lib is None:
        # LIFT_ORACLE_SO: a deliberately mutated copy built by tools/mutate_oracle.py
        # (mutation testing of the pins); never set otherwise
        lib = ctypes.CDLL(os.environ.get("LIFT_ORACLE_SO") or build())
        f32p = ctypes.POINTER(ctypes.c_float)
        f64p = ctypes.POINTER(ctypes.c_double)
        i64 = ctypes.c_int64
        lib.oracle_dot.restype = ctypes.c_double
        lib.oracle_dot.argtypes = [i64, f32p, f32p, f64p]
        lib.oracle_dot_chunked.restype = ctypes.c_double
        lib.oracle_dot_chunked.argtypes = [i64, f32p, f32p, f64p, ctypes.c_int, ctypes.c_int]
        lib.oracle_gemv.restype = None
        lib.oracle_gemv.argtypes = [i64, i64, f32p, f32p, f64p, f64p, ctypes.c_int]
        lib.oracle_gesummv.restype = None
        lib.oracle_gesummv.argtypes = [i64, i64, ctypes.c_float, f32p, ctypes.c_float, f32p, f32p,
                                       f64p, f64p, ctypes.c_int]
        lib.oracle_atax.restype = None
        lib.oracle_atax.argtypes = [i64, i64, f32p, f32p, f64p, f64p, ctypes.c_int]
        lib.oracle_partial_dot.restype = None
        lib.oracle_partial_dot.argtypes = [i64, i64, f32p, f32p, f64p, f64p]
        lib.oracle_partial_dot_listing1_f32.restype = None
        lib.oracle_partial_dot_listing1_f32.argtypes = [i64, f32p, f32p, f32p, ctypes.c_int]
        lib.oracle_dot_listing1_f32.restype = ctypes.c_float
        lib.oracle_dot_listing1_f32.argtypes = [i64, f32p, f32p, ctypes.c_int]
        lib.oracle_sgemv.restype = None
        lib.oracle_sgemv.argtypes = [ctypes.c_int, ctypes.c_int, i64, i64, ctypes.c_float, f32p, i64, f32p,
                                     ctypes.c_float, f32p, f64p, f64p]
        lib.oracle_version.restype = ctypes.c_int
        _lib = lib
    return _lib


def _f32(a) -> np.ndarray:
    a = np.ascontiguousarray(a, dtype=np.float32)
    return a


def _p32(a: np.ndarray):
    return a.ctypes.data_as(ctypes.POINTER(ctypes.c_float))


def _p64(a: np.ndarray):
    return a.ctypes.data_as(ctypes.POINTER(ctypes.c_double))


def default_threads() -> int:
    try:
        return len(os.sched_getaffinity(0))
    except AttributeError:  # pragma: no cover
        return os.cpu_count() or 1


def dot(x, y):
    """(s, mag): s = sum_i x_i*y_i in fp64 (L285)."""
    x, y = _f32(x).ravel(), _f32(y).ravel()
    assert x.shape == y.shape
    mag = ctypes.c_double(0.0)
    s = _load().oracle_dot(x.size, _p32(x), _p32(y), ctypes.byref(mag))
    return float(s), float(mag.value)


def dot_chunked(x, y, chunks: int = 256, threads: int | None = None):
    """(s, mag): the dot over all host cores — fixed chunks folded in order, the
    same bits for every thread count (oracle.h, reading R23)."""
    x, y = _f32(x).ravel(), _f32(y).ravel()
    assert x.shape == y.shape
    mag = ctypes.c_double(0.0)
    s = _load().oracle_dot_chunked(x.size, _p32(x), _p32(y), ctypes.byref(mag), int(chunks),
                                   threads or default_threads())
    return float(s), float(mag.value)


def gemv(A, x, threads: int | None = None):
    """(y, mag) fp64 arrays of length m: y = A x (Table 1 GEMV)."""
    A, x = _f32(A), _f32(x).ravel()
    m, n = A.shape
    assert x.size == n
    y = np.empty(m, np.float64)
    mag = np.empty(m, np.float64)
    _load().oracle_gemv(m, n, _p32(A), _p32(x), _p64(y), _p64(mag), threads or default_threads())
    return y, mag


def gesummv(alpha, A, beta, B, x, threads: int | None = None):
    """(y, mag): y = alpha A x + beta B x with fp32 alpha/beta widened exactly."""
    A, B, x = _f32(A), _f32(B), _f32(x).ravel()
    m, n = A.shape
    assert B.shape == (m, n) and x.size == n
    y = np.empty(m, np.float64)
    mag = np.empty(m, np.float64)
    _load().oracle_gesummv(m, n, ctypes.c_float(alpha), _p32(A), ctypes.c_float(beta), _p32(B),
                           _p32(x), _p64(y), _p64(mag), threads or default_threads())
    return y, mag


def atax(A, x, threads: int | None = None):
    """(y, mag) fp64 arrays of length n: y = A^T (A x)."""
    A, x = _f32(A), _f32(x).ravel()
    m, n = A.shape
    assert x.size == n
    y = np.empty(n, np.float64)
    mag = np.empty(n, np.float64)
    _load().oracle_atax(m, n, _p32(A), _p32(x), _p64(y), _p64(mag), threads or default_threads())
    return y, mag


def partial_dot(x, y, chunk: int = 128):
    """(z, mag): z[k] = sum of the k-th chunk of x*y (Listing 1)."""
    x, y = _f32(x).ravel(), _f32(y).ravel()
    assert x.shape == y.shape
    g = x.size // chunk
    z = np.empty(g, np.float64)
    mag = np.empty(g, np.float64)
    _load().oracle_partial_dot(x.size, chunk, _p32(x), _p32(y), _p64(z), _p64(mag))
    return z, mag


def partial_dot_listing1_f32(x, y, use_fma: bool = True) -> np.ndarray:
    """Listing 1 executed literally in fp32 (paper order); z has n//128 entries."""
    x, y = _f32(x).ravel(), _f32(y).ravel()
    assert x.shape == y.shape
    z = np.empty(x.size // 128, np.float32)
    _load().oracle_partial_dot_listing1_f32(x.size, _p32(x), _p32(y), _p32(z), int(bool(use_fma)))
    return z


def dot_listing1_f32(x, y, use_fma: bool = True) -> float:
    """The whole dot in Listing 1's structure and order, fp32 (reading R26)."""
    x, y = _f32(x).ravel(), _f32(y).ravel()
    assert x.shape == y.shape
    return float(np.float32(_load().oracle_dot_listing1_f32(x.size, _p32(x), _p32(y), int(bool(use_fma)))))


def sgemv(layout, trans, m, n, alpha, A_buf, lda, x, beta, y_in=None):
    """(y, mag): BLAS SGEMV on the stored buffer A_buf (flat fp32), see oracle.h."""
    A_buf = _f32(A_buf).ravel()
    x = _f32(x).ravel()
    ylen = n if trans else m
    yi = _f32(y_in).ravel() if y_in is not None else np.zeros(ylen, np.float32)
    y = np.empty(ylen, np.float64)
    mag = np.empty(ylen, np.float64)
    _load().oracle_sgemv(int(layout), int(trans), m, n, ctypes.c_float(alpha), _p32(A_buf), lda, _p32(x),
                         ctypes.c_float(beta), _p32(yi), _p64(y), _p64(mag))
    return y, mag


def within_tol(got, ref, mag, rtol: float = RTOL, atol: float = ATOL):
    """Elementwise acceptance test; returns (ok, margin) with margin = max |d|/(rtol*mag+atol)."""
    got = np.asarray(got, np.float64)
    ref = np.asarray(ref, np.float64)
    mag = np.asarray(mag, np.float64)
    bound = rtol * mag + atol
    d = np.abs(got - ref)
    if d.size == 0:
        return True, 0.0
    margin = float(np.max(d / bound))
    ok = bool(np.all(d <= bound))
    return ok, margin
