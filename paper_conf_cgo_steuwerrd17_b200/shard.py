"""Row sharding of the hot path across the GPUs of one node (north_star).

One process per GPU; ``torch.distributed`` (backend "nccl" on GPUs) carries
exactly ONE collective per op — the exchange step each op really has:

=========  ==========================================  ======================================
op         partition                                   collective
=========  ==========================================  ======================================
dot        contiguous element slices of x, y           all_reduce(SUM) of one fp32 scalar
GEMV       contiguous row blocks of A; x replicated    all_gather_into_tensor of y blocks
GESUMMV    row blocks of A and B;  x replicated        all_gather_into_tensor of y blocks
ATAX       row blocks of A; x replicated               reduce(SUM, dst) (or all_reduce) of
           (t_r = A_r x is row-local: no exchange)     the partial A_r^T (A_r x)
=========  ==========================================  ======================================

The paper evaluates one GPU only (L999-1007); this layer is new.  Reading R19:
rank r owns rows [floor(r*m/g), floor((r+1)*m/g)).  GEMV/GESUMMV rows use a
canonical per-row summation order (include/lift.h), so the gathered y is
bitwise identical to the single-GPU result.

The per-rank compute is the C-ABI library.  ``local`` lets tests substitute
the per-rank compute (tests/test_shard_gloo.py runs this exact host logic on
CPU with the gloo backend and world_size 2); the product path always uses the
CUDA library and never falls back.
"""
from __future__ import annotations

from dataclasses import dataclass
from typing import Callable, Optional

import torch
import torch.distributed as dist


def partition_rows(m: int, world: int, rank: int) -> tuple[int, int]:
    """Rows [r0, r1) of rank `rank` out of `world` (reading R19)."""
    if world < 1 or not (0 <= rank < world) or m < 0:
        raise ValueError(f"bad partition request m={m} world={world} rank={rank}")
    return (m * rank) // world, (m * (rank + 1)) // world


def shard_sizes(m: int, world: int) -> list[int]:
    return [partition_rows(m, world, r)[1] - partition_rows(m, world, r)[0] for r in range(world)]


@dataclass
class LocalOps:
    """Per-rank compute.  Defaults are the CUDA C-ABI ops."""
    dot: Callable
    gemv: Callable
    gesummv: Callable
    atax: Callable


def cuda_ops() -> LocalOps:
    from . import lift_atax, lift_dot, lift_gemv, lift_gesummv

    return LocalOps(
        dot=lambda x, y, out=None: lift_dot(x, y, out=out),
        gemv=lambda A, x, out=None: lift_gemv(A, x, out=out),
        gesummv=lambda al, A, be, B, x, out=None: lift_gesummv(al, A, be, B, x, out=out),
        atax=lambda A, x, out=None: lift_atax(A, x, out=out),
    )


_default_ops: Optional[LocalOps] = None


def _ops(local: Optional[LocalOps]) -> LocalOps:
    global _default_ops
    if local is not None:
        return local
    if _default_ops is None:
        _default_ops = cuda_ops()
    return _default_ops


def _world(group) -> tuple[int, int]:
    return dist.get_world_size(group), dist.get_rank(group)


def _gather_rows(y_loc: torch.Tensor, m: int, group, out: Optional[torch.Tensor]) -> torch.Tensor:
    """All-gather row blocks of y into a full y (padding only when m % g != 0)."""
    g, r = _world(group)
    sizes = shard_sizes(m, g)
    if y_loc.numel() != sizes[r]:
        raise ValueError(f"rank {r} holds {y_loc.numel()} rows, partition says {sizes[r]}")
    if all(s == sizes[0] for s in sizes):
        y = out if out is not None else torch.empty(m, dtype=y_loc.dtype, device=y_loc.device)
        dist.all_gather_into_tensor(y, y_loc, group=group)
        return y
    pad = max(sizes)
    send = torch.zeros(pad, dtype=y_loc.dtype, device=y_loc.device)
    send[: y_loc.numel()] = y_loc
    buf = torch.empty(pad * g, dtype=y_loc.dtype, device=y_loc.device)
    dist.all_gather_into_tensor(buf, send, group=group)
    y = out if out is not None else torch.empty(m, dtype=y_loc.dtype, device=y_loc.device)
    o = 0
    for k, s in enumerate(sizes):
        y[o:o + s] = buf[k * pad:k * pad + s]
        o += s
    return y


def dot(x_loc: torch.Tensor, y_loc: torch.Tensor, group=None, local: Optional[LocalOps] = None) -> torch.Tensor:
    """sum over ranks of dot(x_loc, y_loc): one all_reduce(SUM) of a 4-byte scalar."""
    s = _ops(local).dot(x_loc, y_loc)
    s = s.reshape(1)
    dist.all_reduce(s, op=dist.ReduceOp.SUM, group=group)
    return s.reshape(())


def gemv(A_loc: torch.Tensor, x: torch.Tensor, m: int, group=None, local: Optional[LocalOps] = None,
         y_loc: Optional[torch.Tensor] = None, out: Optional[torch.Tensor] = None) -> torch.Tensor:
    """y = A x with A row-sharded (rank's rows A_loc); returns the full y on every rank."""
    y_loc = _ops(local).gemv(A_loc, x, out=y_loc)
    return _gather_rows(y_loc, m, group, out)


def gesummv(alpha: float, A_loc: torch.Tensor, beta: float, B_loc: torch.Tensor, x: torch.Tensor, m: int,
            group=None, local: Optional[LocalOps] = None, y_loc: Optional[torch.Tensor] = None,
            out: Optional[torch.Tensor] = None) -> torch.Tensor:
    """y = alpha A x + beta B x with A, B row-sharded; full y on every rank."""
    y_loc = _ops(local).gesummv(alpha, A_loc, beta, B_loc, x, out=y_loc)
    return _gather_rows(y_loc, m, group, out)


def atax(A_loc: torch.Tensor, x: torch.Tensor, group=None, dst: int = 0, allreduce: bool = False,
         local: Optional[LocalOps] = None, out: Optional[torch.Tensor] = None) -> Optional[torch.Tensor]:
    """y = A^T (A x) = sum_r A_r^T (A_r x).  Result on `dst` (None elsewhere),
    or on every rank with allreduce=True."""
    y = _ops(local).atax(A_loc, x, out=out)
    if allreduce:
        dist.all_reduce(y, op=dist.ReduceOp.SUM, group=group)
        return y
    dist.reduce(y, dst=dst, op=dist.ReduceOp.SUM, group=group)
    return y if dist.get_rank(group) == dst else None


# ---------------------------------------------------------------------------
# the same ops with the collective fused into the kernel (include/lift_nvlink.h)
# ---------------------------------------------------------------------------
class FusedGroup:
    """Per-op exchange areas in torch symmetric memory (NVLink peer mappings).

    ``FusedGroup(group)`` must be created collectively; each op/shape gets its
    own area on first use (also a collective: every rank calls the same ops in
    the same order, exactly as with NCCL).  For single-GPU tests pass
    ``areas`` built with :meth:`nvlink.ExchangeArea.simulated`.
    """

    def __init__(self, group=None, areas: Optional[dict] = None, transport: str = "auto"):
        self.group = group
        self.areas = areas if areas is not None else {}
        self.transport = transport  # "symm" | "ipc" | "auto" (symmetric memory, else CUDA IPC)

    def area(self, kind: int, length: int):
        from .nvlink import ExchangeArea

        key = (kind, length)
        if key not in self.areas:
            ex = None
            if self.transport in ("auto", "symm"):
                try:
                    ex = ExchangeArea.symmetric(kind, length, self.group)
                except Exception:  # torch symmetric memory unavailable for this group / layout
                    if self.transport == "symm":
                        raise
            if ex is None:  # both transports map the peers' HBM; IPC also works for ranks sharing a GPU
                ex = ExchangeArea.ipc(kind, length, self.group)
            self.areas[key] = ex
        return self.areas[key]


def fused_self_check(fg: FusedGroup, device: torch.device) -> Optional[str]:
    """Collective: run each fused op once on a small sharded problem with uneven
    shards and compare it with the same op over torch.distributed collectives
    (GEMV / GESUMMV bitwise — same rows, same canonical order; dot / ATAX within
    the north_star tolerance — the two sum the ranks in different orders).
    Returns None when every rank passed, else a one-line reason (the same
    verdict on every rank)."""
    world, rank = _world(fg.group)
    reason = None
    try:
        gen = torch.Generator().manual_seed(20170204)
        nd, m, n = 10007, 1001, 512
        xd, yd = torch.rand(nd, generator=gen) - 0.5, torch.rand(nd, generator=gen) - 0.5
        A, B = torch.rand(m, n, generator=gen) - 0.5, torch.rand(m, n, generator=gen) - 0.5
        x = (torch.rand(n, generator=gen) - 0.5).to(device)
        e0, e1 = partition_rows(nd, world, rank)
        r0, r1 = partition_rows(m, world, rank)
        xl, yl = xd[e0:e1].to(device), yd[e0:e1].to(device)
        Al, Bl = A[r0:r1].contiguous().to(device), B[r0:r1].contiguous().to(device)

        def close(a, b, mag):
            return bool(((a - b).abs() <= 1e-5 * mag + 1e-6).all())

        # every op runs on every rank whatever the earlier verdicts (they are collectives)
        fails = []
        got, want = dot_fused(xl, yl, fg), dot(xl, yl, fg.group)
        if not close(got, want, float((xd * yd).abs().sum())):
            fails.append(f"dot {float(got)} != {float(want)}")
        if not torch.equal(gemv_fused(Al, x, m, fg), gemv(Al, x, m, fg.group)):
            fails.append("gemv all-gather differs")
        if not torch.equal(gesummv_fused(1.5, Al, 1.2, Bl, x, m, fg), gesummv(1.5, Al, 1.2, Bl, x, m, fg.group)):
            fails.append("gesummv all-gather differs")
        got = atax_fused(Al, x, fg, allreduce=True)
        want = atax(Al, x, fg.group, allreduce=True)
        if not close(got, want, (A.abs().T @ (A.abs() @ x.abs().cpu())).to(device)):
            fails.append("atax reduce differs")
        reason = "; ".join(fails) if fails else None
        if device.type == "cuda":
            torch.cuda.synchronize(device)
    except Exception as e:  # setup or launch failure of the fused path
        reason = f"{type(e).__name__}: {str(e).splitlines()[0] if str(e) else ''}"
    flag = torch.tensor([0 if reason is None else 1], device=device, dtype=torch.int32)
    dist.all_reduce(flag, op=dist.ReduceOp.MAX, group=fg.group)
    if int(flag.item()) and reason is None:
        reason = "failed on another rank"
    return reason


def dot_fused(x_loc: torch.Tensor, y_loc: torch.Tensor, fg: FusedGroup, out=None) -> torch.Tensor:
    """dot with the all-reduce inside the kernel: identical bits on every rank."""
    from .nvlink import EXCH_DOT, lift_dot_allreduce

    return lift_dot_allreduce(x_loc, y_loc, fg.area(EXCH_DOT, 0), out=out)


def gemv_fused(A_loc: torch.Tensor, x: torch.Tensor, m: int, fg: FusedGroup, row0: Optional[int] = None,
               out=None) -> torch.Tensor:
    """GEMV whose rows are stored straight into every rank's y (fused all-gather)."""
    from .nvlink import EXCH_GATHER, lift_gemv_allgather

    ex = fg.area(EXCH_GATHER, m)
    if row0 is None:
        row0 = partition_rows(m, ex.world, ex.rank)[0]
    return lift_gemv_allgather(A_loc, x, row0, m, ex, out=out)


def gesummv_fused(alpha: float, A_loc: torch.Tensor, beta: float, B_loc: torch.Tensor, x: torch.Tensor, m: int,
                  fg: FusedGroup, row0: Optional[int] = None, out=None) -> torch.Tensor:
    from .nvlink import EXCH_GATHER, lift_gemv_allgather

    ex = fg.area(EXCH_GATHER, m)
    if row0 is None:
        row0 = partition_rows(m, ex.world, ex.rank)[0]
    return lift_gemv_allgather(A_loc, x, row0, m, ex, out=out, B=B_loc, alpha=alpha, beta=beta)


def atax_fused(A_loc: torch.Tensor, x: torch.Tensor, fg: FusedGroup, dst: int = 0, allreduce: bool = False,
               out=None) -> Optional[torch.Tensor]:
    """ATAX whose partial A_r^T (A_r x) is reduced over ranks inside the kernel."""
    from .nvlink import EXCH_REDUCE, lift_atax_reduce

    ex = fg.area(EXCH_REDUCE, x.numel())
    y = lift_atax_reduce(A_loc, x, ex, dst=-1 if allreduce else dst, out=out)
    return y if (allreduce or ex.rank == dst) else None
