"""C-ABI library: loads, exports every symbol include/*.h declares, and its
host-side validation returns the documented status codes before touching
CUDA.  Pointers here are fake integers: no error path dereferences them."""
import ctypes
import subprocess

import pytest

import paper_conf_cgo_steuwerrd17_b200 as lift
from paper_conf_cgo_steuwerrd17_b200 import _lib

L = lift.lib()
OK, NULL, SIZE, MIS, ALIAS, WS, CUDA = range(7)

P = 1 << 20  # fake, 256-B aligned "device" addresses far apart
A_, B_, X_, Y_, W_ = P * 16, P * 64, P * 128, P * 160, P * 192


def _gpu() -> bool:
    import torch

    return torch.cuda.is_available()


def test_library_exports_every_header_symbol():
    names = _lib.header_functions()
    assert {"lift_dot", "lift_gemv", "lift_gesummv", "lift_atax"} <= set(names)
    out = subprocess.run(["nm", "-D", "--defined-only", lift.library_path()], capture_output=True, text=True,
                         check=True).stdout
    exported = {line.split()[-1] for line in out.splitlines() if " T " in line}
    missing = [n for n in names if n not in exported]
    assert not missing, missing
    for n in names:
        assert hasattr(L, n)
    assert set(names) == set(_lib.SIGNATURES)


def test_exports_nothing_else():
    out = subprocess.run(["nm", "-D", "--defined-only", lift.library_path()], capture_output=True, text=True,
                         check=True).stdout
    exported = {line.split()[-1] for line in out.splitlines() if " T " in line}
    assert {e for e in exported if e.startswith("lift_")} == set(_lib.header_functions())


def test_sm100a_cubin_only():
    out = subprocess.run(["cuobjdump", "--list-elf", lift.library_path()], capture_output=True, text=True).stdout
    assert "sm_100a" in out
    for bad in ("sm_90", "sm_80", "sm_103"):
        assert bad not in out


def test_version_and_strerror():
    assert L.lift_version() >> 16 == 2
    for s in range(7):
        msg = L.lift_strerror(s).decode()
        assert msg.startswith("LIFT_")
    assert L.lift_strerror(99).decode() == "unknown lift status"


def test_workspace_sizes():
    assert L.lift_dot_workspace_bytes(0) >= 16 + 4 * 148
    assert L.lift_dot_workspace_bytes(1 << 31) == L.lift_dot_workspace_bytes(1)
    w = L.lift_atax_workspace_bytes(8192, 8192)
    assert w >= 8192 * 4 + 148 * 8192 * 4
    assert L.lift_atax_workspace_bytes(-1, 5) == 0


# ---------------------------------------------------------------- dot
def test_dot_validation():
    ws_ok = L.lift_dot_workspace_bytes(100)
    assert L.lift_dot(-1, X_, Y_, W_ + ws_ok + 64, W_, ws_ok, None) == SIZE
    assert L.lift_dot(100, None, Y_, P * 300, W_, ws_ok, None) == NULL
    assert L.lift_dot(100, X_, Y_, None, W_, ws_ok, None) == NULL
    assert L.lift_dot(100, X_ + 2, Y_, P * 300, W_, ws_ok, None) == MIS
    assert L.lift_dot(100, X_, Y_, P * 300, None, ws_ok, None) == WS
    assert L.lift_dot(100, X_, Y_, P * 300, W_, ws_ok - 4, None) == WS
    assert L.lift_dot(100, X_, Y_, P * 300, W_ + 4, ws_ok, None) == WS
    assert L.lift_dot(100, X_, Y_, X_ + 8, W_, ws_ok, None) == ALIAS  # result inside x
    assert L.lift_dot(100, X_, Y_, W_ + 16, W_, ws_ok, None) == ALIAS  # result inside workspace
    assert L.lift_dot(100, X_, Y_, P * 300, Y_ + 64, ws_ok, None) == ALIAS  # workspace over y


# ---------------------------------------------------------------- GEMV family
def test_gemv_validation():
    assert L.lift_gemv(-1, 4, A_, X_, Y_, None) == SIZE
    assert L.lift_gemv(4, -1, A_, X_, Y_, None) == SIZE
    assert L.lift_gemv(1 << 40, 1 << 40, A_, X_, Y_, None) == SIZE  # m*n*4 overflows
    assert L.lift_gemv(4, 4, None, X_, Y_, None) == NULL
    assert L.lift_gemv(4, 4, A_, None, Y_, None) == NULL
    assert L.lift_gemv(4, 4, A_, X_, None, None) == NULL
    assert L.lift_gemv(4, 4, A_ + 1, X_, Y_, None) == MIS
    assert L.lift_gemv(4, 4, A_, X_, Y_ + 2, None) == MIS
    assert L.lift_gemv(4, 4, A_, X_, A_ + 60, None) == ALIAS
    assert L.lift_gemv(4, 4, A_, X_, X_ - 4, None) == ALIAS
    # m == 0 is a no-op that never touches CUDA (even with NULL pointers)
    assert L.lift_gemv(0, 4, None, None, None, None) == OK
    # aligned but only 4-byte aligned is accepted (scalar path): must reach CUDA
    if not _gpu():  # on a GPU box a valid call would launch on the fake pointers
        st = L.lift_gemv(4, 3, A_ + 4, X_ + 4, Y_ + 4, None)
        assert st in (OK, CUDA)


def test_gesummv_validation():
    assert L.lift_gesummv(4, 4, 1.0, A_, 1.0, None, X_, Y_, None) == NULL
    assert L.lift_gesummv(4, 4, 1.0, A_, 1.0, B_ + 2, X_, Y_, None) == MIS
    assert L.lift_gesummv(4, 4, 1.0, A_, 1.0, B_, X_, B_ + 4, None) == ALIAS
    assert L.lift_gesummv(0, 4, 1.0, None, 1.0, None, None, None, None) == OK


def test_tuned_validation():
    assert L.lift_gemv_tuned(-1, 4, A_, X_, Y_, 8, 1, 0, -1, 4, None) == SIZE
    assert L.lift_gesummv_tuned(4, 4, 1.0, A_, 1.0, B_, X_, A_, 8, 1, 0, -1, 4, None) == ALIAS
    ws = L.lift_atax_workspace_bytes(64, 512)
    assert L.lift_atax_fused_tuned(-1, 512, A_, X_, Y_, W_, ws, 0, -1, None) == SIZE
    assert L.lift_atax_fused_tuned(64, 512, A_, X_, None, W_, ws, 0, -1, None) == NULL
    assert L.lift_atax_fused_tuned(64, 512, A_, X_, Y_, W_, ws - 16, 0, -1, None) == WS
    assert L.lift_atax_fused_tuned(64, 512, A_, X_ + 4, Y_, W_, ws, 0, -1, None) == SIZE  # fused needs 16-B
    assert L.lift_atax_fused_tuned(64, 510, A_, X_, Y_, W_, ws, 0, -1, None) == SIZE  # and n % 4 == 0
    assert L.lift_atax_fused_tuned(64, 512, A_, X_, A_, W_, ws, 0, -1, None) == ALIAS


def test_atax_fused_grid_validation():
    import ctypes

    b, c = ctypes.c_int(0), ctypes.c_int(0)
    assert L.lift_atax_fused_grid(64, 512, None, ctypes.byref(c)) == NULL
    assert L.lift_atax_fused_grid(0, 512, ctypes.byref(b), ctypes.byref(c)) == SIZE  # no rows: no launch shape
    assert L.lift_atax_fused_grid(64, 510, ctypes.byref(b), ctypes.byref(c)) == SIZE  # n % 4
    assert L.lift_atax_fused_grid(64, 16388, ctypes.byref(b), ctypes.byref(c)) == SIZE  # no whole-float4 slices
    if not _gpu():
        assert L.lift_atax_fused_grid(64, 512, ctypes.byref(b), ctypes.byref(c)) == CUDA


# ---------------------------------------------------------------- ATAX
def test_atax_validation():
    m, n = 64, 32
    ws = L.lift_atax_workspace_bytes(m, n)
    assert L.lift_atax(-2, n, A_, X_, Y_, W_, ws, None) == SIZE
    assert L.lift_atax(m, n, None, X_, Y_, W_, ws, None) == NULL
    assert L.lift_atax(m, n, A_, X_, None, W_, ws, None) == NULL
    assert L.lift_atax(m, n, A_, X_ + 1, Y_, W_, ws, None) == MIS
    assert L.lift_atax(m, n, A_, X_, Y_, None, ws, None) == WS
    assert L.lift_atax(m, n, A_, X_, Y_, W_, ws - 1, None) == WS
    assert L.lift_atax(m, n, A_, X_, Y_, W_ + 8, ws, None) == WS
    assert L.lift_atax(m, n, A_, X_, A_ + 128, W_, ws, None) == ALIAS
    assert L.lift_atax(m, n, A_, X_, Y_, A_, ws, None) == ALIAS
    if not _gpu():  # valid args: reaches CUDA (no device here)
        assert L.lift_atax(m, n, A_, X_, Y_, W_ + 8 * 1024 * 1024, ws, None) in (OK, CUDA)
    assert L.lift_atax_algo_run(7, m, n, A_, X_, Y_, W_, ws, None) == SIZE
    # fused needs n % 4 == 0 and 16-B alignment: refused up front
    assert L.lift_atax_algo_run(1, m, 33, A_, X_, Y_, W_, L.lift_atax_workspace_bytes(m, 33), None) == SIZE
    assert L.lift_atax(m, 0, A_, X_, Y_, W_, L.lift_atax_workspace_bytes(m, 0), None) == OK


def test_valid_call_without_gpu_fails_loudly():
    import torch

    if torch.cuda.is_available():
        pytest.skip("a GPU is present")
    st = L.lift_gemv(4, 4, A_, X_, Y_, None)
    assert st == CUDA
    assert "cuda" in L.lift_last_cuda_error().decode().lower() or "device" in L.lift_last_cuda_error().decode().lower()
    with pytest.raises(lift.LiftError):
        _lib.check(st)


def test_python_binding_rejects_cpu_tensors():
    import torch

    A = torch.zeros(4, 4)
    x = torch.zeros(4)
    with pytest.raises(ValueError, match="no CPU path"):
        lift.lift_gemv(A, x)
    with pytest.raises(TypeError):
        lift.lift_gemv(A.double(), x)


def test_ctypes_signatures_match_header_arity():
    import re

    import glob

    txt = "".join(open(f).read() for f in sorted(glob.glob(_lib._build.INCLUDE + "/*.h")))
    txt = re.sub(r"/\*.*?\*/", "", txt, flags=re.S)
    for name, (_, args) in _lib.SIGNATURES.items():
        m = re.search(r"\b" + name + r"\s*\(([^)]*)\)", txt)
        assert m, name
        params = [p for p in m.group(1).split(",") if p.strip() and p.strip() != "void"]
        assert len(params) == len(args), (name, params)
    assert ctypes.sizeof(ctypes.c_size_t) == 8


def test_listing1_validation():
    assert L.lift_partial_dot(-1, X_, Y_, Y_ + (1 << 24), 1, None) == SIZE
    assert L.lift_partial_dot(256, X_, Y_, P * 300, 2, None) == SIZE  # contract must be 0 or 1
    assert L.lift_partial_dot(100, None, None, None, 1, None) == OK  # no work group: nothing to do
    assert L.lift_partial_dot(256, None, Y_, P * 300, 1, None) == NULL
    assert L.lift_partial_dot(256, X_ + 1, Y_, P * 300, 1, None) == MIS
    assert L.lift_partial_dot(256, X_, Y_, X_ + 4, 1, None) == ALIAS
    ws = L.lift_dot_listing1_workspace_bytes(1000)
    assert ws >= 2 * 8 * 4
    assert L.lift_dot_listing1(1000, X_, Y_, P * 300, W_, ws - 1, 1, None) == WS
    assert L.lift_dot_listing1(1000, X_, Y_, W_ + 8, W_, ws, 1, None) == ALIAS
    assert L.lift_dot_listing1(1000, X_, Y_, None, W_, ws, 1, None) == NULL


def test_sgemv_validation():
    assert L.lift_sgemv_workspace_bytes(0, 0, 100, 50) == 0          # row-major, no transpose: no workspace
    assert L.lift_sgemv_workspace_bytes(0, 1, 100, 50) > 0
    assert L.lift_sgemv_workspace_bytes(1, 0, 100, 50) > 0           # column-major = transposed rows
    assert L.lift_sgemv_workspace_bytes(1, 1, 100, 50) == 0
    assert L.lift_sgemv(2, 0, 4, 4, 1.0, A_, 4, X_, 0.0, Y_, None, 0, None) == SIZE
    assert L.lift_sgemv(0, 0, 4, 4, 1.0, A_, 3, X_, 0.0, Y_, None, 0, None) == SIZE   # lda < n
    assert L.lift_sgemv(1, 1, 4, 6, 1.0, A_, 3, X_, 0.0, Y_, None, 0, None) == SIZE   # col-major lda < m
    assert L.lift_sgemv(0, 0, 4, 4, 1.0, None, 4, X_, 0.0, Y_, None, 0, None) == NULL
    assert L.lift_sgemv(0, 1, 4, 4, 1.0, A_, 4, X_, 0.0, Y_, None, 0, None) == WS
    assert L.lift_sgemv(0, 0, 4, 4, 1.0, A_, 8, X_, 0.0, A_ + 4 * 9, None, 0, None) == ALIAS
    assert L.lift_sgemv(0, 0, 0, 4, 1.0, None, 4, None, 0.0, None, None, 0, None) == OK


def test_nvlink_validation():
    peers = P * 400
    ws = L.lift_dot_workspace_bytes(100)
    assert L.lift_exchange_bytes(0, 0, 8) >= 2048 + 2 * 64 * 4
    assert L.lift_exchange_bytes(1, 65536, 8) >= 2 * 65536 * 4
    assert L.lift_exchange_bytes(2, 8192, 8) >= 2 * 8 * 8192 * 4
    assert L.lift_exchange_bytes(3, 10, 8) == 0 and L.lift_exchange_bytes(0, 1, 65) == 0
    assert L.lift_dot_allreduce(100, X_, Y_, P * 300, W_, ws, peers, 0, 0, None) == SIZE      # world 0
    assert L.lift_dot_allreduce(100, X_, Y_, P * 300, W_, ws, peers, 2, 2, None) == SIZE      # rank >= world
    assert L.lift_dot_allreduce(100, X_, Y_, P * 300, W_, ws, None, 0, 2, None) == NULL
    assert L.lift_dot_allreduce(100, X_, Y_, P * 300, W_, ws, peers + 4, 0, 2, None) == MIS
    assert L.lift_gemv_allgather(10, 4, A_, X_, 95, 100, Y_, W_, 256, peers, 0, 2, None) == SIZE  # rows past m_total
    assert L.lift_gemv_allgather(10, 4, A_, X_, 0, 100, A_, W_, 256, peers, 0, 2, None) == ALIAS
    assert L.lift_gemv_allgather(10, 4, A_, X_, 0, 100, Y_, W_, 8, peers, 0, 2, None) == WS
    assert L.lift_gesummv_allgather(10, 4, 1.0, A_, 1.0, None, X_, 0, 10, Y_, W_, 256, peers, 0, 1, None) == NULL
    wsa = L.lift_atax_workspace_bytes(64, 512)
    assert L.lift_atax_reduce(64, 512, A_, X_, Y_, W_, wsa, peers, 0, 2, 2, 0, None) == SIZE      # dst >= world
    assert L.lift_atax_reduce(64, 510, A_, X_, Y_, W_, wsa, peers, 0, 2, 0, 0, None) == SIZE     # n % 4
    assert L.lift_atax_reduce(64, 512, A_, X_ + 2, Y_, W_, wsa, peers, 0, 2, 0, 0, None) == MIS  # not 4-byte
    assert L.lift_atax_reduce(64, 512, A_, X_ + 4, Y_, W_, wsa, peers, 0, 2, 0, 0, None) == SIZE  # not 16-byte
    assert L.lift_atax_reduce(64, 512, A_, None, Y_, W_, wsa, peers, 0, 2, 0, 0, None) == NULL
    assert L.lift_atax_reduce(64, 512, A_, X_, Y_, A_ + 256, wsa, peers, 0, 2, 0, 0, None) == ALIAS  # ws in A
    assert L.lift_gemv_allgather(10, 4, A_, X_, 0, 100, Y_, A_ + 16, 256, peers, 0, 2, None) == ALIAS  # ticket in A
    assert L.lift_gemv_allgather(10, 4, A_, X_, 0, 100, Y_, X_, 256, peers, 0, 2, None) == ALIAS       # ticket on x
    assert L.lift_gesummv_allgather(10, 4, 1.0, A_, 1.0, B_, X_, 0, 10, Y_, B_, 256, peers, 0, 1, None) == ALIAS


def test_host_entry_validation():
    assert L.lift_gemv_host(-1, 4, A_, X_, Y_, A_, X_, Y_, None) == SIZE
    assert L.lift_gemv_host(4, 4, None, X_, Y_, A_, X_, Y_, None) == NULL
    assert L.lift_gemv_host(4, 4, A_, X_, Y_, A_, A_ + 8, Y_, None) == ALIAS      # device buffers overlap
    assert L.lift_gesummv_host(4, 4, 1.0, A_, 1.0, B_, X_, Y_, A_, A_, X_, Y_, None) == ALIAS
    assert L.lift_dot_host(8, X_, Y_, None, X_, Y_, W_, W_ + 64, 256, None) == NULL
    assert L.lift_atax_host(0, 0, None, None, None, None, None, None, None, 0, None) == OK
