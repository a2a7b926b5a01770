"""Sharded ops with the collective fused into the kernel (include/lift_nvlink.h, NEXT-2).

Each rank's kernel writes its results straight into every destination
rank's exchange area (NVLink peer stores), publishes a flag, and the
receivers combine contributions in rank order.  An :class:`ExchangeArea`
holds one rank's view: its own area, the device array of every rank's area
pointers.  Calls on one area must happen in the same order on every rank; the
call counter (epoch) lives in the area itself on the device, so a sequence of
fused calls can be captured in a CUDA graph and replayed.

* :meth:`ExchangeArea.symmetric` — one area per rank from torch symmetric
  memory (multi-GPU, one process per GPU).
* :meth:`ExchangeArea.simulated` — ``world`` areas on ONE device sharing one
  peer table: the exact kernels and protocol with "peers" in the same
  HBM, for tests on a single GPU (the ranks' kernels run concurrently on
  separate streams).
"""
from __future__ import annotations

import torch

from . import _check_len, _check_out, _check_tensor, _same_device, _stream, _workspace
from ._lib import check, lib

EXCH_DOT, EXCH_GATHER, EXCH_REDUCE = 0, 1, 2


class ExchangeArea:
    def __init__(self, kind: int, length: int, area: torch.Tensor, peers: torch.Tensor, rank: int, world: int):
        self.kind, self.length = kind, length
        self.area, self.peers = area, peers  # keep the allocations alive
        self.rank, self.world = rank, world

    @staticmethod
    def nbytes(kind: int, length: int, world: int) -> int:
        b = lib().lift_exchange_bytes(kind, length, world)
        if b == 0:
            raise ValueError(f"bad exchange request kind={kind} length={length} world={world}")
        return b

    @classmethod
    def symmetric(cls, kind: int, length: int, group=None) -> "ExchangeArea":
        """This rank's area in torch symmetric memory (collective call over `group`)."""
        import torch.distributed as dist
        import torch.distributed._symmetric_memory as symm_mem

        world, rank = dist.get_world_size(group), dist.get_rank(group)
        dev = torch.device("cuda", torch.cuda.current_device())
        nb = cls.nbytes(kind, length, world)
        area = symm_mem.empty(nb, dtype=torch.uint8, device=dev)
        area.zero_()
        hdl = symm_mem.rendezvous(area, group if group is not None else dist.group.WORLD)
        peers = torch.tensor(list(hdl.buffer_ptrs), dtype=torch.int64, device=dev)
        torch.cuda.synchronize(dev)
        dist.barrier(group)
        return cls(kind, length, area, peers, rank, world)

    @classmethod
    def ipc(cls, kind: int, length: int, group=None) -> "ExchangeArea":
        """This rank's area from cudaMalloc, shared with CUDA IPC handles (collective).

        The transport for ranks that torch symmetric memory refuses (e.g. several
        processes on one GPU); across GPUs the opened handles map the peers' HBM
        over NVLink (cudaIpcMemLazyEnablePeerAccess)."""
        import torch.distributed as dist
        from cuda.bindings import runtime as rt

        def ok(res):
            err = res[0] if isinstance(res, tuple) else res
            if int(err) != 0:
                raise RuntimeError(f"CUDA runtime error {err}")
            return res[1] if isinstance(res, tuple) and len(res) > 1 else None

        world, rank = dist.get_world_size(group), dist.get_rank(group)
        dev_index = torch.cuda.current_device()
        ok(rt.cudaSetDevice(dev_index))
        nb = cls.nbytes(kind, length, world)
        ptr = int(ok(rt.cudaMalloc(nb)))
        ok(rt.cudaMemset(ptr, 0, nb))
        ok(rt.cudaDeviceSynchronize())
        handle = ok(rt.cudaIpcGetMemHandle(ptr))
        mine = bytes(handle.reserved)
        handles = [None] * world
        dist.all_gather_object(handles, mine, group=group)
        ptrs, opened = [], []
        for r, hb in enumerate(handles):
            if r == rank:
                ptrs.append(ptr)
                continue
            h = rt.cudaIpcMemHandle_t()
            h.reserved = hb
            p = int(ok(rt.cudaIpcOpenMemHandle(h, rt.cudaIpcMemLazyEnablePeerAccess)))
            ptrs.append(p)
            opened.append(p)
        peers = torch.tensor(ptrs, dtype=torch.int64, device=torch.device("cuda", dev_index))
        torch.cuda.synchronize()
        dist.barrier(group)
        ex = cls(kind, length, None, peers, rank, world)
        ex._ipc = (rt, ptr, opened)
        return ex

    def close(self) -> None:
        """Release an IPC area (collective: peers must be done with it)."""
        ipc = getattr(self, "_ipc", None)
        if ipc is not None:
            rt, ptr, opened = ipc
            for p in opened:
                rt.cudaIpcCloseMemHandle(p)
            rt.cudaFree(ptr)
            self._ipc = None

    @classmethod
    def simulated(cls, kind: int, length: int, world: int, device) -> list["ExchangeArea"]:
        """`world` areas on one device, one peer table: rank r's view is element r."""
        nb = cls.nbytes(kind, length, world)
        areas = [torch.zeros(nb, dtype=torch.uint8, device=device) for _ in range(world)]
        peers = torch.tensor([a.data_ptr() for a in areas], dtype=torch.int64, device=device)
        return [cls(kind, length, areas[r], peers, r, world) for r in range(world)]


def _check_area(ex: ExchangeArea, kind: int, length: int) -> None:
    """The kernels size their stores by the call's shape: the area must have been
    made for this kind and length (the device-side extent is not visible to them)."""
    if ex.kind != kind or (kind != EXCH_DOT and ex.length != length):
        raise ValueError(f"exchange area made for kind {ex.kind} length {ex.length}, the call needs kind {kind} "
                         f"length {length}")


def workspace_bytes(op: str, m: int = 0, n: int = 0) -> int:
    """Workspace bytes of one call (allocate zeroed, reuse across calls)."""
    L = lib()
    if op == "dot":
        return L.lift_dot_workspace_bytes(n)
    if op in ("gemv", "gesummv"):
        return 256
    if op == "atax":
        return L.lift_atax_workspace_bytes(m, n)
    raise ValueError(op)


def lift_dot_allreduce(x: torch.Tensor, y: torch.Tensor, ex: ExchangeArea, out: torch.Tensor | None = None,
                       workspace: torch.Tensor | None = None):
    """Sum over ranks of dot(x_r, y_r); the same bits on every rank.

    Pass `out` and `workspace` (zeroed uint8) when ranks share one device:
    allocating inside the call may synchronise the device while a peer rank's
    kernel is waiting for this one."""
    _check_tensor(x, "x", 1)
    _check_tensor(y, "y", 1)
    dev = _same_device(x, y)
    _check_len(y, "y", x.numel())
    _check_area(ex, EXCH_DOT, 0)
    if out is None:
        out = torch.empty((), dtype=torch.float32, device=dev)
    _check_out(out, "out", 1, dev)
    L = lib()
    n = x.numel()
    with torch.cuda.device(dev):
        ws = workspace if workspace is not None else _workspace(f"dotar{ex.rank}", dev,
                                                                L.lift_dot_workspace_bytes(n), zero=True)
        check(L.lift_dot_allreduce(n, x.data_ptr(), y.data_ptr(), out.data_ptr(), ws.data_ptr(), ws.numel(),
                                   ex.peers.data_ptr(), ex.rank, ex.world, _stream(dev)))
    return out


def lift_gemv_allgather(A: torch.Tensor, x: torch.Tensor, row0: int, m_total: int, ex: ExchangeArea,
                        out: torch.Tensor | None = None, B: torch.Tensor | None = None, alpha: float = 1.0,
                        beta: float = 0.0, workspace: torch.Tensor | None = None):
    """Rows [row0, row0 + A.shape[0]) computed here; the full y on every rank.
    With B given: GESUMMV (alpha A x + beta B x)."""
    _check_tensor(A, "A", 2)
    _check_tensor(x, "x", 1)
    dev = _same_device(A, x)
    _check_area(ex, EXCH_GATHER, m_total)
    m, n = A.shape
    _check_len(x, "x", n)
    if B is not None:
        _check_tensor(B, "B", 2)
        _same_device(A, B)
        if tuple(B.shape) != (m, n):
            raise ValueError(f"B has shape {tuple(B.shape)}, A {(m, n)}")
    if out is None:
        out = torch.empty(m_total, dtype=torch.float32, device=dev)
    _check_out(out, "out", m_total, dev)
    L = lib()
    with torch.cuda.device(dev):
        ws = workspace if workspace is not None else _workspace(f"gather{ex.rank}", dev, 256, zero=True)
        if B is None:
            st = L.lift_gemv_allgather(m, n, A.data_ptr(), x.data_ptr(), row0, m_total, out.data_ptr(), ws.data_ptr(),
                                       ws.numel(), ex.peers.data_ptr(), ex.rank, ex.world,
                                       _stream(dev))
        else:
            st = L.lift_gesummv_allgather(m, n, float(alpha), A.data_ptr(), float(beta), B.data_ptr(), x.data_ptr(),
                                          row0, m_total, out.data_ptr(), ws.data_ptr(), ws.numel(),
                                          ex.peers.data_ptr(), ex.rank, ex.world, _stream(dev))
        check(st)
    return out


def lift_atax_reduce(A: torch.Tensor, x: torch.Tensor, ex: ExchangeArea, dst: int = -1,
                     out: torch.Tensor | None = None, blocks: int = 0, workspace: torch.Tensor | None = None):
    """y = sum over ranks of A_r^T (A_r x) on `dst` (-1: every rank)."""
    _check_tensor(A, "A", 2)
    _check_tensor(x, "x", 1)
    dev = _same_device(A, x)
    m, n = A.shape
    _check_len(x, "x", n)
    _check_area(ex, EXCH_REDUCE, n)
    if out is None:
        out = torch.empty(n, dtype=torch.float32, device=dev)
    _check_out(out, "out", n, dev)
    L = lib()
    with torch.cuda.device(dev):
        ws = workspace if workspace is not None else _workspace(f"ataxr{ex.rank}", dev,
                                                                L.lift_atax_workspace_bytes(m, n), zero=True)
        check(L.lift_atax_reduce(m, n, A.data_ptr(), x.data_ptr(), out.data_ptr(), ws.data_ptr(), ws.numel(),
                                 ex.peers.data_ptr(), ex.rank, ex.world, dst, blocks, _stream(dev)))
    return out
