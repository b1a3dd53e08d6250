"""Slab decomposition of an iterated 3D stencil across ranks.

The global grid (N0, N1, N2) is cut along dimension 0 (the slowest, z) into
contiguous slabs, one per rank (one process per GPU).  Every state buffer of
a rank holds its owned planes plus ``ghost = max(pad_lo[0], pad_hi[0])`` ghost
planes on each side.  A time step (iterate) is:

  1. boundary output planes [0, g) and [n-g, n) of the slab — they read the
     ghosts received during the previous step;
  2. the freshly computed boundary planes go to the neighbour ranks' ghost
     planes (NCCL send/recv over NVLink on a side stream, ``DistExchange``);
  3. concurrently, the interior output planes [g, n-g) — they need no ghosts.

Global boundaries are handled by pad against the GLOBAL extent inside the
kernels (stencil_plan_set_slab); WRAP in z turns the chain into a ring.  Each
output point is produced by the same kernel code as on one GPU, so the
decomposed result is bitwise equal to the single-GPU result.

The orchestration (partition, neighbour pairing, exchange order, region
split) is plain torch.distributed and is exercised on CPU with gloo in the
tests; on GPUs the compute callback is ``Plan.apply_region`` (libstencil.so).
``LocalExchange`` runs G slabs inside one process on one device ("virtual
slab" mode) with device-to-device copies, for single-GPU verification.
"""
from __future__ import annotations

from typing import Callable, List, Optional, Sequence, Tuple

import torch
import torch.distributed as dist

WRAP = 2


def partition(n0: int, world: int) -> List[Tuple[int, int]]:
    """Balanced contiguous split of n0 planes over ``world`` ranks."""
    if world < 1 or n0 < world:
        raise ValueError(f"cannot split {n0} planes over {world} ranks")
    return [(r * n0 // world, (r + 1) * n0 // world) for r in range(world)]


def neighbours(rank: int, world: int, wrap: bool) -> Tuple[Optional[int], Optional[int]]:
    """(lower, upper) neighbour ranks along z; None at a non-periodic global edge."""
    lo = rank - 1 if rank > 0 else (world - 1 if wrap else None)
    hi = rank + 1 if rank < world - 1 else (0 if wrap else None)
    return lo, hi


class DistExchange:
    """Ghost-plane exchange through torch.distributed point-to-point ops.

    For buffer ``b`` of ``n + 2g`` planes: owned planes [g, 2g) go to the lower
    neighbour's upper ghosts, owned planes [n, n+g) go to the upper neighbour's
    lower ghosts.  Ops are posted as [send low -> lo, recv hi-ghost <- hi,
    send high -> hi, recv lo-ghost <- lo]: with two ranks on a ring both
    neighbours are the same peer, and this order pairs each send with the right
    ghost (NCCL matches same-peer p2p ops in posting order)."""

    def __init__(self, rank: int, world: int, n: int, ghost: int, wrap: bool, group=None):
        self.rank, self.world, self.n, self.g = rank, world, n, ghost
        self.lo, self.hi = neighbours(rank, world, wrap)
        self.group = group
        if world == 1:
            self.lo = self.hi = None
            self.self_wrap = wrap
        else:
            self.self_wrap = False

    def post(self, buf: torch.Tensor) -> list:
        n, g = self.n, self.g
        if self.self_wrap:        # one rank on a ring: ghosts are its own far planes
            buf[0:g].copy_(buf[n:n + g])
            buf[n + g:n + 2 * g].copy_(buf[g:2 * g])
            return []
        ops = []
        if self.lo is not None:
            ops.append(dist.P2POp(dist.isend, buf[g:2 * g], self.lo, self.group, tag=0))
        if self.hi is not None:
            ops.append(dist.P2POp(dist.irecv, buf[n + g:n + 2 * g], self.hi, self.group, tag=0))
        if self.hi is not None:
            ops.append(dist.P2POp(dist.isend, buf[n:n + g], self.hi, self.group, tag=1))
        if self.lo is not None:
            ops.append(dist.P2POp(dist.irecv, buf[0:g], self.lo, self.group, tag=1))
        if not ops:
            return []
        return dist.batch_isend_irecv(ops)


def slab_step(compute: Callable[[int, int], None], exchange_post: Callable[[], list],
              n: int, g: int, on_comm: Callable[[Callable[[], list]], list] = None,
              wait: Callable[[list], None] = None):
    """One time step: boundary planes, then (exchange || interior).

    ``compute(a, b)`` writes output planes [a, b) of the slab;
    ``exchange_post()`` posts the ghost exchange of the freshly written output
    buffer and returns its works; ``on_comm`` runs the post on the side stream;
    ``wait`` joins the works before the next step's boundary compute."""
    if n <= 2 * g:
        compute(0, n)
        works = on_comm(exchange_post) if on_comm else exchange_post()
        return works
    compute(0, g)
    compute(n - g, n)
    works = on_comm(exchange_post) if on_comm else exchange_post()
    compute(g, n - g)
    return works


class SlabPlan:
    """One rank's slab of a global 3D stencil (CUDA, libstencil.so).

    ``global_extents`` is (N0, N1, N2); the remaining arguments are those of
    :class:`Plan`.  Buffers have shape ``(n_local + 2*ghost, N1, N2)``."""

    def __init__(self, global_extents: Sequence[int], rank: int, world: int, size=3, pad=None, kind="clamp",
                 pad_value: float = 0.0, op="weighted", weights=None, params=(), group=None,
                 device: Optional[int] = None, exchange=None, exchange_factory=None):
        from .plan import Plan, KINDS, _kind
        self.global_extents = tuple(int(e) for e in global_extents)
        self.rank, self.world = rank, world
        self.z0, self.z1 = partition(self.global_extents[0], world)[rank]
        self.n = self.z1 - self.z0
        ext = (self.n,) + self.global_extents[1:]
        self.plan = Plan(ext, size, 1, pad, None, kind, pad_value, op, weights, params, device)
        self.g = max(self.plan.pad_lo[0], self.plan.pad_hi[0])
        if self.n < max(self.g, 1):
            raise ValueError("slab thinner than the ghost width")
        self.plan.set_slab(self.z0, self.global_extents[0], self.g)
        self.wrap = self.plan.kind[0] == WRAP
        factory = exchange_factory if exchange_factory is not None else DistExchange
        self.exchange = exchange if exchange is not None else factory(rank, world, self.n, self.g, self.wrap, group)
        self.comm = torch.cuda.Stream(device=self.plan.device)
        self.alloc_shape = self.plan.alloc_extents

    def empty(self) -> torch.Tensor:
        return torch.empty(self.alloc_shape, dtype=torch.float32, device=f"cuda:{self.plan.device}")

    def scatter(self, global_grid: torch.Tensor) -> torch.Tensor:
        """Local buffer with the owned planes of ``global_grid`` (ghosts unset)."""
        buf = self.empty()
        buf[self.g:self.g + self.n].copy_(global_grid[self.z0:self.z1])
        return buf

    def owned(self, buf: torch.Tensor) -> torch.Tensor:
        return buf[self.g:self.g + self.n]

    def _on_comm(self, post):
        cur = torch.cuda.current_stream()
        self.comm.wait_stream(cur)
        with torch.cuda.stream(self.comm):
            works = post()
        return works

    def _join(self, works):
        for w in works:
            w.wait()                       # on the comm stream
        torch.cuda.current_stream().wait_stream(self.comm)

    def iterate(self, state: Sequence[torch.Tensor], n_steps: int, aux: Sequence[torch.Tensor] = ()) -> int:
        """n time steps with the rotation of stencil_iterate (A21);
        returns the index of the state buffer holding the newest grid."""
        op = self.plan.op
        acoustic = op == 4
        ri = 1 if acoustic else 0
        self._join(self._on_comm(lambda: self.exchange.post(state[ri])))
        for _ in range(n_steps):
            if acoustic:
                dst = 1 - ri
                ins = (state[dst], state[ri])
            else:
                dst = 1 - ri
                ins = (state[ri],) + tuple(aux)
            out = state[dst]
            works = slab_step(lambda a, b: self.plan.apply_region(*ins, out=out, begin=a, end=b),
                              lambda: self.exchange.post(out), self.n, self.g, on_comm=self._on_comm)
            self._join(works)
            ri = dst
        return ri


class LocalExchange:
    """Virtual-slab exchange: all slabs live in one process (one device); the
    ghost planes are filled by device-to-device copies from the neighbour
    slab's buffer registered under the same key."""

    def __init__(self, slabs: List["SlabPlan"]):
        self.slabs = slabs

    def fill(self, bufs: List[torch.Tensor]):
        G = len(self.slabs)
        for r, s in enumerate(self.slabs):
            lo, hi = neighbours(r, G, s.wrap)
            n, g = s.n, s.g
            if lo is not None:
                sl = self.slabs[lo]
                bufs[r][0:g].copy_(bufs[lo][sl.n:sl.n + g])
            if hi is not None:
                bufs[r][n + g:n + 2 * g].copy_(bufs[hi][g:2 * g])


def virtual_slab_iterate(global_extents, world: int, state_global: Sequence[torch.Tensor], n_steps: int,
                         aux_global: Sequence[torch.Tensor] = (), **plan_kw) -> List[torch.Tensor]:
    """Run G slabs on the current device (no process group) and return the
    reassembled global state (newest grid last for ACOUSTIC, else [newest])."""
    slabs = [SlabPlan(global_extents, r, world, exchange=_NoExchange(), **plan_kw) for r in range(world)]
    ex = LocalExchange(slabs)
    nst = len(state_global)
    bufs = [[s.scatter(state_global[k]) if k < nst else s.empty() for k in range(2)] for s in slabs]
    if nst == 1:
        pass
    auxs = [[s.scatter(a) for a in aux_global] for s in slabs]
    acoustic = slabs[0].plan.op == 4
    ri = 1 if acoustic else 0
    ex.fill([b[ri] for b in bufs])
    for _ in range(n_steps):
        dst = 1 - ri
        for s, b, a in zip(slabs, bufs, auxs):
            ins = (b[dst], b[ri]) if acoustic else (b[ri],) + tuple(a)
            s.plan.apply(*ins, out=b[dst])
        ex.fill([b[dst] for b in bufs])
        ri = dst
    out = []
    order = [1 - ri, ri] if acoustic else [ri]
    for k in order:
        out.append(torch.cat([s.owned(b[k]) for s, b in zip(slabs, bufs)], 0))
    return out


class _NoExchange:
    def post(self, buf):
        return []
