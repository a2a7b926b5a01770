"""ctypes loader for liblift.so (include/lift.h).  Argument marshalling only.

The library is built in-tree for sm_100a (``build.py``).  If it is missing or
older than its sources it is (re)built with nvcc; if that fails, importing the
binding raises — there is no fallback path of any kind.
"""
from __future__ import annotations

import ctypes
import os
import re
import threading

from . import build as _build

_lock = threading.Lock()
_lib = None

LIFT_OK = 0
LIFT_ERR_NULL_PTR = 1
LIFT_ERR_BAD_SIZE = 2
LIFT_ERR_MISALIGNED = 3
LIFT_ERR_ALIAS = 4
LIFT_ERR_WORKSPACE = 5
LIFT_ERR_CUDA = 6

LIFT_ATAX_AUTO = 0
LIFT_ATAX_FUSED = 1
LIFT_ATAX_TWOPASS = 2

i64 = ctypes.c_int64
u64 = ctypes.c_uint64
vp = ctypes.c_void_p
f32 = ctypes.c_float
i32 = ctypes.c_int
sz = ctypes.c_size_t

# name -> (restype, argtypes); mirrors include/lift.h and include/lift_tuning.h
SIGNATURES = {
    "lift_dot_workspace_bytes": (sz, [i64]),
    "lift_dot": (i32, [i64, vp, vp, vp, vp, sz, vp]),
    "lift_gemv": (i32, [i64, i64, vp, vp, vp, vp]),
    "lift_gesummv": (i32, [i64, i64, f32, vp, f32, vp, vp, vp, vp]),
    "lift_atax_workspace_bytes": (sz, [i64, i64]),
    "lift_atax": (i32, [i64, i64, vp, vp, vp, vp, sz, vp]),
    "lift_atax_algo_run": (i32, [i32, i64, i64, vp, vp, vp, vp, sz, vp]),
    "lift_sgemv_workspace_bytes": (sz, [i32, i32, i64, i64]),
    "lift_sgemv": (i32, [i32, i32, i64, i64, f32, vp, i64, vp, f32, vp, vp, sz, vp]),
    "lift_partial_dot": (i32, [i64, vp, vp, vp, i32, vp]),
    "lift_dot_listing1_workspace_bytes": (sz, [i64]),
    "lift_dot_listing1": (i32, [i64, vp, vp, vp, vp, sz, i32, vp]),
    "lift_exchange_bytes": (sz, [i32, i64, i32]),
    "lift_dot_allreduce": (i32, [i64, vp, vp, vp, vp, sz, vp, i32, i32, vp]),
    "lift_gemv_allgather": (i32, [i64, i64, vp, vp, i64, i64, vp, vp, sz, vp, i32, i32, vp]),
    "lift_gesummv_allgather": (i32, [i64, i64, f32, vp, f32, vp, vp, i64, i64, vp, vp, sz, vp, i32, i32, vp]),
    "lift_atax_reduce": (i32, [i64, i64, vp, vp, vp, vp, sz, vp, i32, i32, i32, i32, vp]),
    "lift_dot_host": (i32, [i64, vp, vp, vp, vp, vp, vp, vp, sz, vp]),
    "lift_gemv_host": (i32, [i64, i64, vp, vp, vp, vp, vp, vp, vp]),
    "lift_gesummv_host": (i32, [i64, i64, f32, vp, f32, vp, vp, vp, vp, vp, vp, vp, vp]),
    "lift_atax_host": (i32, [i64, i64, vp, vp, vp, vp, vp, vp, vp, sz, vp]),
    "lift_strerror": (ctypes.c_char_p, [i32]),
    "lift_last_cuda_error": (ctypes.c_char_p, []),
    "lift_version": (i32, []),
    "lift_gemv_tuned": (i32, [i64, i64, vp, vp, vp, i32, i32, i32, i32, i32, vp]),
    "lift_gesummv_tuned": (i32, [i64, i64, f32, vp, f32, vp, vp, vp, i32, i32, i32, i32, i32, vp]),
    "lift_atax_fused_tuned": (i32, [i64, i64, vp, vp, vp, vp, sz, i32, i32, vp]),
    "lift_atax_fused_grid": (i32, [i64, i64, vp, vp]),
}


class LiftError(RuntimeError):
    def __init__(self, status: int, msg: str):
        super().__init__(f"{msg} (status {status})")
        self.status = status


def lib():
    """The loaded liblift.so with argtypes set (built on first use if needed)."""
    global _lib
    if _lib is None:
        with _lock:
            if _lib is None:
                path = _build.build()
                L = ctypes.CDLL(path)
                for name, (res, args) in SIGNATURES.items():
                    fn = getattr(L, name)
                    fn.restype = res
                    fn.argtypes = args
                _lib = L
    return _lib


def library_path() -> str:
    return _build.SO


def check(status: int) -> None:
    if status != LIFT_OK:
        L = lib()
        msg = L.lift_strerror(status).decode()
        if status == LIFT_ERR_CUDA:
            msg += ": " + L.lift_last_cuda_error().decode()
        raise LiftError(status, msg)


def header_functions(paths=None) -> list[str]:
    """Names of the functions declared in include/*.h (for export checks)."""
    if paths is None:
        inc = os.path.join(_build.ROOT, "include")
        paths = [os.path.join(inc, f) for f in sorted(os.listdir(inc)) if f.endswith(".h")]
    names = []
    for p in paths:
        txt = open(p).read()
        txt = re.sub(r"/\*.*?\*/", "", txt, flags=re.S)
        for m in re.finditer(r"\b(lift_[a-z0-9_]+)\s*\(", txt):
            if m.group(1) not in names:
                names.append(m.group(1))
    return names
