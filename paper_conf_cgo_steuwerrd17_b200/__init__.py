"""B200-native Lift hot path: the fused zip -> map(x) -> reduce(+) kernel
(Steuwer, Remmelg, Dubach, CGO 2017) for dot, GEMV, GESUMMV and ATAX.

Thin Python binding over the C ABI in ``include/lift.h`` (``liblift.so``):
every step of the path runs in the library's CUDA kernels; this module only
checks tensors, allocates outputs / workspaces with torch, and passes raw
device pointers plus ``torch.cuda.current_stream()``.  The function names are
the C names.  Inputs must be fp32, contiguous CUDA tensors on one device.

Sharded (multi-GPU) variants live in :mod:`paper_conf_cgo_steuwerrd17_b200.shard`.
"""
from __future__ import annotations

import contextlib
import threading

import torch

from ._lib import (LIFT_ATAX_AUTO, LIFT_ATAX_FUSED, LIFT_ATAX_TWOPASS, LiftError,  # noqa: F401
                   check, lib, library_path)

__all__ = ["lift_dot", "lift_gemv", "lift_gesummv", "lift_atax", "lift_gemv_tuned", "lift_gesummv_tuned",
           "lift_atax_fused_tuned", "lift_atax_fused_grid",
           "lift_partial_dot", "lift_dot_listing1", "lift_sgemv",
           "LiftError", "lib", "library_path", "KERNELS_PER_CALL"]

# kernels each entry point enqueues (for the bench's gpu_launches count)
KERNELS_PER_CALL = {"lift_dot": 1, "lift_gemv": 1, "lift_gesummv": 1, "lift_atax_fused": 1, "lift_atax_twopass": 3}

_ws_lock = threading.Lock()
_ws_cache: dict = {}


def _check_tensor(t: torch.Tensor, name: str, dim: int | None = None) -> None:
    if not isinstance(t, torch.Tensor):
        raise TypeError(f"{name} must be a torch.Tensor")
    if t.dtype != torch.float32:
        raise TypeError(f"{name} must be float32 (got {t.dtype})")
    if t.device.type != "cuda":
        raise ValueError(f"{name} must be a CUDA tensor (got {t.device}); there is no CPU path")
    if not t.is_contiguous():
        raise ValueError(f"{name} must be contiguous")
    if dim is not None and t.dim() != dim:
        raise ValueError(f"{name} must be {dim}-D (got shape {tuple(t.shape)})")


def _same_device(*ts: torch.Tensor) -> torch.device:
    d = ts[0].device
    for t in ts[1:]:
        if t.device != d:
            raise ValueError(f"tensors on different devices: {d} vs {t.device}")
    return d


def _check_out(out: torch.Tensor, name: str, numel: int, device: torch.device) -> None:
    """An output the kernels write: fp32, contiguous, on `device`, exactly `numel`
    elements (the C ABI takes a bare pointer and cannot check its extent)."""
    _check_tensor(out, name)
    if out.device != device:
        raise ValueError(f"{name} is on {out.device}, the inputs on {device}")
    if out.numel() != numel:
        raise ValueError(f"{name} has {out.numel()} elements, the result has {numel}")


def _check_len(t: torch.Tensor, name: str, numel: int) -> None:
    if t.numel() != numel:
        raise ValueError(f"{name} has {t.numel()} elements, expected {numel}")


_NULL_CTX = contextlib.nullcontext()


def _on(device: torch.device):
    """torch.cuda.device(device), skipped when it is already current (the
    common case: switching devices costs a few microseconds per call)."""
    return _NULL_CTX if device.index == torch.cuda.current_device() else torch.cuda.device(device)


# the raw handle of the current stream without building a torch.cuda.Stream
# object (0.07 instead of 2.2 us per call, tools/binding_profile.py)
_raw_stream = getattr(torch._C, "_cuda_getCurrentRawStream", None)


def _stream(device: torch.device) -> int:
    if _raw_stream is not None:
        return _raw_stream(device.index)
    return torch.cuda.current_stream(device).cuda_stream


def _capture_id(stream: int) -> int:
    """Id of the CUDA-graph capture sequence `stream` is in (unique per process)."""
    from cuda.bindings import runtime as rt
    err, _status, cid = rt.cudaStreamGetCaptureInfo(stream)[:3]
    if int(err) != 0:
        raise RuntimeError(f"cudaStreamGetCaptureInfo failed: {err}")
    return int(cid)


def _workspace(kind: str, device: torch.device, nbytes: int, zero: bool) -> torch.Tensor:
    """Per-(kind, device, stream, capture) cached workspace, grown on demand.

    The dot and ATAX workspaces start with counters that must be zero before
    first use; they are allocated with torch.zeros and every call leaves them
    zero again.  A workspace first allocated while a CUDA graph is being
    captured is zeroed only when that graph replays, so it is keyed by the
    capture sequence and never handed to eager calls or to another graph."""
    stream = _stream(device)
    cid = _capture_id(stream) if torch.cuda.is_current_stream_capturing() else 0
    key = (kind, device.index, stream, cid)
    with _ws_lock:
        ws = _ws_cache.get(key)
        if ws is None or ws.numel() < nbytes:
            alloc = torch.zeros if zero else torch.empty
            ws = alloc(max(nbytes, 256), dtype=torch.uint8, device=device)
            _ws_cache[key] = ws
        return ws


def lift_dot(x: torch.Tensor, y: torch.Tensor, out: torch.Tensor | None = None) -> torch.Tensor:
    """0-d fp32 CUDA tensor sum_i x_i*y_i  (Listing 1)."""
    _check_tensor(x, "x", 1)
    _check_tensor(y, "y", 1)
    dev = _same_device(x, y)
    if x.numel() != y.numel():
        raise ValueError("x and y must have the same length")
    if out is None:
        out = torch.empty((), dtype=torch.float32, device=dev)
    _check_out(out, "out", 1, dev)
    L = lib()
    n = x.numel()
    nbytes = L.lift_dot_workspace_bytes(n)
    with _on(dev):
        ws = _workspace("dot", dev, nbytes, zero=True)
        check(L.lift_dot(n, x.data_ptr(), y.data_ptr(), out.data_ptr(), ws.data_ptr(), ws.numel(), _stream(dev)))
    return out


def lift_gemv(A: torch.Tensor, x: torch.Tensor, out: torch.Tensor | None = None) -> torch.Tensor:
    """y = A x, A (m, n) row-major fp32  (Table 1 GEMV, L1030)."""
    _check_tensor(A, "A", 2)
    _check_tensor(x, "x", 1)
    dev = _same_device(A, x)
    m, n = A.shape
    if x.numel() != n:
        raise ValueError(f"x has {x.numel()} elements, A has {n} columns")
    if out is None:
        out = torch.empty(m, dtype=torch.float32, device=dev)
    _check_tensor(out, "out", 1)
    _check_out(out, "out", m, dev)
    with _on(dev):
        check(lib().lift_gemv(m, n, A.data_ptr(), x.data_ptr(), out.data_ptr(), _stream(dev)))
    return out


def lift_gemv_tuned(A, x, out=None, wpr=0, rg=0, blocks=0, xsmem=-1, lb=0):
    """lift_gemv with an explicit launch configuration (include/lift_tuning.h)."""
    _check_tensor(A, "A", 2)
    _check_tensor(x, "x", 1)
    dev = _same_device(A, x)
    m, n = A.shape
    _check_len(x, "x", n)
    if out is None:
        out = torch.empty(m, dtype=torch.float32, device=dev)
    _check_out(out, "out", m, dev)
    with _on(dev):
        check(lib().lift_gemv_tuned(m, n, A.data_ptr(), x.data_ptr(), out.data_ptr(), wpr, rg, blocks, xsmem, lb,
                                    _stream(dev)))
    return out


def lift_gesummv(alpha: float, A: torch.Tensor, beta: float, B: torch.Tensor, x: torch.Tensor,
                 out: torch.Tensor | None = None) -> torch.Tensor:
    """y = alpha A x + beta B x  (Table 1 GESUMMV, L1031); alpha/beta passed as fp32."""
    _check_tensor(A, "A", 2)
    _check_tensor(B, "B", 2)
    _check_tensor(x, "x", 1)
    dev = _same_device(A, B, x)
    m, n = A.shape
    if tuple(B.shape) != (m, n) or x.numel() != n:
        raise ValueError("shape mismatch")
    if out is None:
        out = torch.empty(m, dtype=torch.float32, device=dev)
    _check_tensor(out, "out", 1)
    _check_out(out, "out", m, dev)
    with _on(dev):
        check(lib().lift_gesummv(m, n, float(alpha), A.data_ptr(), float(beta), B.data_ptr(), x.data_ptr(),
                                 out.data_ptr(), _stream(dev)))
    return out


def lift_gesummv_tuned(alpha, A, beta, B, x, out=None, wpr=0, rg=0, blocks=0, xsmem=-1, lb=0):
    _check_tensor(A, "A", 2)
    _check_tensor(B, "B", 2)
    _check_tensor(x, "x", 1)
    dev = _same_device(A, B, x)
    m, n = A.shape
    if tuple(B.shape) != (m, n):
        raise ValueError("shape mismatch")
    _check_len(x, "x", n)
    if out is None:
        out = torch.empty(m, dtype=torch.float32, device=dev)
    _check_out(out, "out", m, dev)
    with _on(dev):
        check(lib().lift_gesummv_tuned(m, n, float(alpha), A.data_ptr(), float(beta), B.data_ptr(), x.data_ptr(),
                                       out.data_ptr(), wpr, rg, blocks, xsmem, lb, _stream(dev)))
    return out


_ALGOS = {"auto": LIFT_ATAX_AUTO, "fused": LIFT_ATAX_FUSED, "twopass": LIFT_ATAX_TWOPASS}


def lift_atax(A: torch.Tensor, x: torch.Tensor, out: torch.Tensor | None = None, algo: str = "auto") -> torch.Tensor:
    """y = A^T (A x)  (Table 1 ATAX, L1029).  algo: "auto" | "fused" | "twopass"."""
    _check_tensor(A, "A", 2)
    _check_tensor(x, "x", 1)
    dev = _same_device(A, x)
    m, n = A.shape
    if x.numel() != n:
        raise ValueError(f"x has {x.numel()} elements, A has {n} columns")
    if out is None:
        out = torch.empty(n, dtype=torch.float32, device=dev)
    _check_tensor(out, "out", 1)
    _check_out(out, "out", n, dev)
    L = lib()
    nbytes = L.lift_atax_workspace_bytes(m, n)
    with _on(dev):
        ws = _workspace("atax", dev, nbytes, zero=True)
        check(L.lift_atax_algo_run(_ALGOS[algo], m, n, A.data_ptr(), x.data_ptr(), out.data_ptr(), ws.data_ptr(),
                                   ws.numel(), _stream(dev)))
    return out


def lift_atax_fused_tuned(A: torch.Tensor, x: torch.Tensor, out: torch.Tensor | None = None, nst: int = 0,
                          cyclic: int = -1) -> torch.Tensor:
    """lift_atax(algo="fused") with the ring depth / row assignment overridden (lift_tuning.h)."""
    _check_tensor(A, "A", 2)
    _check_tensor(x, "x", 1)
    dev = _same_device(A, x)
    m, n = A.shape
    if x.numel() != n:
        raise ValueError(f"x has {x.numel()} elements, A has {n} columns")
    if out is None:
        out = torch.empty(n, dtype=torch.float32, device=dev)
    _check_tensor(out, "out", 1)
    _check_out(out, "out", n, dev)
    L = lib()
    nbytes = L.lift_atax_workspace_bytes(m, n)
    with _on(dev):
        ws = _workspace("atax", dev, nbytes, zero=True)
        check(L.lift_atax_fused_tuned(m, n, A.data_ptr(), x.data_ptr(), out.data_ptr(), ws.data_ptr(), ws.numel(),
                                      nst, cyclic, _stream(dev)))
    return out


def lift_atax_fused_grid(m: int, n: int) -> tuple[int, int]:
    """(blocks, cluster size) of lift_atax's single pass for an m x n matrix on the
    current device (lift_tuning.h); launches nothing."""
    import ctypes

    b, c = ctypes.c_int(0), ctypes.c_int(0)
    check(lib().lift_atax_fused_grid(m, n, ctypes.byref(b), ctypes.byref(c)))
    return b.value, c.value


def lift_partial_dot(x: torch.Tensor, y: torch.Tensor, out: torch.Tensor | None = None,
                     contract: bool = True) -> torch.Tensor:
    """Listing 1 (L391-401) in the paper's exact order: z[k] for k < n//128."""
    _check_tensor(x, "x", 1)
    _check_tensor(y, "y", 1)
    dev = _same_device(x, y)
    if x.numel() != y.numel():
        raise ValueError("x and y must have the same length")
    n = x.numel()
    if out is None:
        out = torch.empty(n // 128, dtype=torch.float32, device=dev)
    _check_tensor(out, "out", 1)
    _check_out(out, "out", n // 128, dev)
    with _on(dev):
        check(lib().lift_partial_dot(n, x.data_ptr(), y.data_ptr(), out.data_ptr(), int(bool(contract)), _stream(dev)))
    return out


def lift_dot_listing1(x: torch.Tensor, y: torch.Tensor, out: torch.Tensor | None = None,
                      contract: bool = True) -> torch.Tensor:
    """The whole dot in Listing 1's structure, iterated to one value (reading R26)."""
    _check_tensor(x, "x", 1)
    _check_tensor(y, "y", 1)
    dev = _same_device(x, y)
    if x.numel() != y.numel():
        raise ValueError("x and y must have the same length")
    if out is None:
        out = torch.empty((), dtype=torch.float32, device=dev)
    _check_out(out, "out", 1, dev)
    L = lib()
    n = x.numel()
    with _on(dev):
        ws = _workspace("listing1", dev, L.lift_dot_listing1_workspace_bytes(n), zero=False)
        check(L.lift_dot_listing1(n, x.data_ptr(), y.data_ptr(), out.data_ptr(), ws.data_ptr(), ws.numel(),
                                  int(bool(contract)), _stream(dev)))
    return out


def lift_sgemv(alpha: float, A: torch.Tensor, x: torch.Tensor, beta: float = 0.0, y: torch.Tensor | None = None,
               trans: bool = False, layout: str = "row", lda: int | None = None, shape=None) -> torch.Tensor:
    """BLAS SGEMV: y = alpha * op(A) x + beta * y (CLBlast contract, NEXT-4).

    A is the stored buffer: a 2-D tensor whose rows are the matrix's rows
    (layout="row") or columns (layout="col"), possibly wider than the matrix
    (lda = A.shape[1] unless given).  `shape` = (m, n) of the logical matrix
    (default: from A).  y is updated in place when given (beta != 0 reads it).
    """
    _check_tensor(A, "A", 2)
    _check_tensor(x, "x", 1)
    dev = _same_device(A, x)
    lay = {"row": 0, "col": 1}[layout]
    if shape is None:
        shape = tuple(A.shape) if lay == 0 else (A.shape[1], A.shape[0])
    m, n = shape
    ld = A.shape[1] if lda is None else lda
    rows, cols = (m, n) if lay == 0 else (n, m)
    if rows > 0 and cols > 0 and A.numel() < (rows - 1) * ld + cols:
        raise ValueError(f"A holds {A.numel()} elements, a {rows} x {cols} matrix with lda {ld} needs "
                         f"{(rows - 1) * ld + cols}")
    ylen = n if trans else m
    if y is None:
        if beta != 0.0:
            raise ValueError("beta != 0 needs y")
        y = torch.empty(ylen, dtype=torch.float32, device=dev)
    _check_tensor(y, "y", 1)
    if y.device != dev:
        raise ValueError(f"y is on {y.device}, A and x on {dev}")
    if y.numel() != ylen or x.numel() != (m if trans else n):
        raise ValueError("x / y length does not match op(A)")
    L = lib()
    need = L.lift_sgemv_workspace_bytes(lay, int(bool(trans)), m, n)
    with _on(dev):
        ws = _workspace("sgemv", dev, need, zero=True) if need else None
        check(L.lift_sgemv(lay, int(bool(trans)), m, n, float(alpha), A.data_ptr(), ld, x.data_ptr(), float(beta),
                           y.data_ptr(), ws.data_ptr() if ws is not None else None, ws.numel() if ws is not None else 0,
                           _stream(dev)))
    return y


# ---------------------------------------------------------------------------
# end to end from host buffers (include/lift_host.h)
# ---------------------------------------------------------------------------
def _check_host(t: torch.Tensor, name: str) -> None:
    if t.dtype != torch.float32 or t.device.type != "cpu" or not t.is_contiguous():
        raise ValueError(f"{name} must be a contiguous fp32 CPU tensor (pinned for asynchronous copies)")


def lift_host_call(op: str, host: dict, dev: dict, alpha: float = 1.0, beta: float = 0.0) -> None:
    """Enqueue one op from host buffers on the current stream: H2D copies of the
    inputs into the caller's device buffers, the kernels, the D2H copy of the
    result (host["out"]).  Synchronise the stream before reading host["out"]."""
    L = lib()
    for k, t in host.items():
        _check_host(t, k)
    device = next(iter(dev.values())).device
    for k, t in host.items():  # the device buffers the copies land in: same extents
        if k not in dev:
            raise ValueError(f"no device buffer for {k}")
        _check_out(dev[k], f"dev[{k!r}]", t.numel(), device)
    s = _stream(device)
    with torch.cuda.device(device):
        if op == "dot":
            n = host["x"].numel()
            ws = _workspace("dot", device, L.lift_dot_workspace_bytes(n), zero=True)
            st = L.lift_dot_host(n, host["x"].data_ptr(), host["y"].data_ptr(), host["out"].data_ptr(),
                                 dev["x"].data_ptr(), dev["y"].data_ptr(), dev["out"].data_ptr(), ws.data_ptr(),
                                 ws.numel(), s)
        elif op == "gemv":
            m, n = host["A"].shape
            st = L.lift_gemv_host(m, n, host["A"].data_ptr(), host["x"].data_ptr(), host["out"].data_ptr(),
                                  dev["A"].data_ptr(), dev["x"].data_ptr(), dev["out"].data_ptr(), s)
        elif op == "gesummv":
            m, n = host["A"].shape
            st = L.lift_gesummv_host(m, n, float(alpha), host["A"].data_ptr(), float(beta), host["B"].data_ptr(),
                                     host["x"].data_ptr(), host["out"].data_ptr(), dev["A"].data_ptr(),
                                     dev["B"].data_ptr(), dev["x"].data_ptr(), dev["out"].data_ptr(), s)
        elif op == "atax":
            m, n = host["A"].shape
            ws = _workspace("atax", device, L.lift_atax_workspace_bytes(m, n), zero=True)
            st = L.lift_atax_host(m, n, host["A"].data_ptr(), host["x"].data_ptr(), host["out"].data_ptr(),
                                  dev["A"].data_ptr(), dev["x"].data_ptr(), dev["out"].data_ptr(), ws.data_ptr(),
                                  ws.numel(), s)
        else:
            raise ValueError(op)
        check(st)
