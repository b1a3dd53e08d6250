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


def deep_halo_iterate(n_steps: int, k: int, r: int, n: int, g: int, extension, compute, post, on_comm, join,
                      acoustic: bool, ri: int, aux=(), compute2=None) -> int:
    """The time-step schedule of a slab with ghosts of g = r*k planes (k = 1:
    the plain per-step exchange).  ``compute(src, dst, a, b)`` writes output
    planes [a, b) (slab-local, may reach into the ghosts) of state ``dst`` from
    state ``src``; ``post(grids)`` posts the ghost exchange of the listed state
    indices / tensors and returns its works; ``on_comm`` runs a post on the
    side stream, ``join`` waits for its works; ``extension(e)`` is the output
    range reaching e planes into the ghosts on the sides that have a
    neighbour.  ``compute2(src, dst, a, b)`` (optional) advances TWO steps in
    one pass on output planes [a, b) (stencil_apply2_region): a block then runs
    its steps in pairs — a pair's region is that of its second step, the first
    step's wider region being implied — and an odd block starts with one
    single step.  Returns the index of the newest state."""
    first = [ri]
    if k > 1:
        first += [1 - ri] if acoustic else list(aux)
    join(on_comm(lambda: post(first)))
    t = 0
    while t < n_steps:
        kb = min(k, n_steps - t)
        if compute2 is not None and kb >= 2:
            j = 1
            if kb % 2:                      # odd block: one single extended step first
                a, b = extension((kb - 1) * r)
                compute(ri, 1 - ri, a, b)
                ri = 1 - ri
                j = 2
            while j <= kb:
                dst = 1 - ri
                if j + 1 < kb:              # steps j, j+1 before the block's last pair
                    a, b = extension((kb - j - 1) * r)
                    compute2(ri, dst, a, b)
                else:                       # the block's last two steps: boundary, (exchange || interior)
                    src = ri
                    works = slab_step(lambda a, b: compute2(src, dst, a, b), lambda: post([dst]), n, g,
                                      on_comm=on_comm)
                    join(works)
                ri = dst
                j += 2
            t += kb
            continue
        for j in range(1, kb + 1):
            dst = 1 - ri
            if j < kb:
                a, b = extension((kb - j) * r)
                compute(ri, dst, a, b)
            else:
                # the block's last step: exactly the owned planes, boundary
                # first, then (exchange || interior); Acoustic with k > 1 also
                # exchanges the new u^{n-1} (the grid just read as u^n)
                grids = [dst, ri] if (acoustic and k > 1) else [dst]
                src = ri
                works = slab_step(lambda a, b: compute(src, dst, a, b), lambda: post(grids), n, g, on_comm=on_comm)
                join(works)
            ri = dst
        t += kb
    return ri


class SlabPlan:
    """One rank's slab of a global 3D stencil (CUDA, libstencil.so).

    ``global_extents`` is (N0, N1, N2); the remaining arguments are those of
    :class:`Plan`.  Buffers have shape ``(n_local + 2*ghost, N1, N2)``."""

    def __init__(self, global_extents: Sequence[int], rank: int, world: int, size=3, pad=None, kind="clamp",
                 pad_value: float = 0.0, op="weighted", weights=None, params=(), group=None,
                 device: Optional[int] = None, exchange=None, exchange_factory=None, depth: int = 1):
        from .plan import Plan
        self.global_extents = tuple(int(e) for e in global_extents)
        self.rank, self.world = rank, world
        self.z0, self.z1 = partition(self.global_extents[0], world)[rank]
        self.n = self.z1 - self.z0
        ext = (self.n,) + self.global_extents[1:]
        self.plan = Plan(ext, size, 1, pad, None, kind, pad_value, op, weights, params, device)
        # deep halos (NEXT-3): ghosts of r*depth planes, exchanged every depth steps
        if depth < 1:
            raise ValueError("halo depth must be >= 1")
        self.r = max(self.plan.pad_lo[0], self.plan.pad_hi[0])
        self.depth = depth
        self.g = self.r * depth
        if self.n < max(self.g, 1):
            raise ValueError("slab thinner than the ghost width")
        self.exchanges = 0      # ghost exchanges posted (each: every exchanged grid, both neighbours)
        self.plan.set_slab(self.z0, self.global_extents[0], self.g)
        self.wrap = self.plan.kind[0] == WRAP
        factory = exchange_factory if exchange_factory is not None else DistExchange
        self.exchange = exchange if exchange is not None else factory(rank, world, self.n, self.g, self.wrap, group)
        self.comm = torch.cuda.Stream(device=self.plan.device)
        self.alloc_shape = self.plan.alloc_extents
        self.epoch = 0          # fused-halo step counter (flag values only grow)

    def _iterate_fused(self, state, n_steps, aux, fused, ri, acoustic):
        # the initial ghosts came through ``exchange``; the flags already hold
        # self.epoch on every rank (all ranks run the same number of steps)
        return _iterate_fused_impl(self, state, n_steps, aux, fused, ri, acoustic)

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

    def _post(self, bufs):
        self.exchanges += 1
        works = []
        for b in bufs:
            works += self.exchange.post(b)
        return works

    def extension(self, e: int) -> Tuple[int, int]:
        """Output plane range [lo, hi) of a step whose region reaches ``e``
        planes into the ghosts on every side that has a neighbour (global,
        non-periodic edges are never extended: pad is applied there)."""
        lo_nb, hi_nb = neighbours(self.rank, self.world, self.wrap)
        if self.world == 1 and self.wrap:
            lo_nb = hi_nb = 0
        return (-e if lo_nb is not None else 0), (self.n + e if hi_nb is not None else self.n)

    def iterate(self, state: Sequence[torch.Tensor], n_steps: int, aux: Sequence[torch.Tensor] = (),
                fused: Optional[FusedHalo] = None) -> int:
        """n time steps with the rotation of stencil_iterate (A21);
        returns the index of the state buffer holding the newest grid.  With
        ``fused`` the ghosts travel by peer stores from the boundary kernel
        (stencil_apply_region_put) instead of NCCL.

        Deep halos (``depth`` k > 1, NEXT-3; the overlapped-tiling rule of
        P:739-791 applied in time): ghosts hold g = r*k planes; a block of
        kb <= k steps starts from fully exchanged ghosts, step j of the block
        computes the owned planes plus (kb - j)*r ghost planes on each side
        that has a neighbour (the neighbour computes the same planes with the
        same kernel code: bitwise identical), and the block's last step
        computes exactly the owned planes, boundary first, with the exchange of
        g planes overlapped with its interior.  Acoustic exchanges both of its
        grids per block (its point-wise u^{n-1} is read in the extended
        region); Hotspot's fixed grid P is exchanged once.  One exchange per k
        time steps instead of one per step."""
        op = self.plan.op
        acoustic = op == 4
        ri = 1 if acoustic else 0
        if fused is not None:
            if self.depth > 1:
                raise ValueError("the fused halo path exchanges every step (depth 1)")
            self._join(self._on_comm(lambda: self._post([state[ri]])))
            return self._iterate_fused(state, n_steps, aux, fused, ri, acoustic)

        def compute(src, dst, a, b):
            ins = (state[dst], state[src]) if acoustic else (state[src],) + tuple(aux)
            self.plan.apply_region(*ins, out=state[dst], begin=a, end=b)

        def post(grids):
            return self._post([state[i] if isinstance(i, int) else i for i in grids])

        compute2 = None
        if op == 0 and self.plan.time_block == 2 and self.r == 1:
            # weighted 7-point star: two steps per pass (K2R) inside the blocks
            def compute2(src, dst, a, b):
                self.plan.apply2_region(state[src], out=state[dst], begin=a, end=b)

        return deep_halo_iterate(n_steps, self.depth, self.r, self.n, self.g, self.extension, compute, post,
                                 self._on_comm, self._join, acoustic, ri, aux, compute2=compute2)


def _iterate_fused_impl(slab, state, n_steps, aux, fused, ri, acoustic):
    stream = torch.cuda.current_stream()
    for _ in range(n_steps):
        dst = 1 - ri
        ins = (state[dst], state[ri]) if acoustic else (state[ri],) + tuple(aux)
        slab.epoch += 1
        fused_step(slab, fused, ins, state[dst], dst, slab.epoch, stream)
        ri = dst
    return ri


class FusedHalo:
    """Peer view for the fused halo put: the boundary-plane kernel
    stores its planes into the neighbours' ghost planes through NVLink peer
    pointers and raises their flags; no NCCL call on the data path.

    ``peer_state[k][r]`` is rank r's state buffer k (a tensor this rank can
    address: a symmetric-memory peer view on real GPUs, the tensor itself in
    virtual mode); ``peer_flags[r]`` is rank r's int32[2] flag array
    ([written by the lower neighbour, written by the upper neighbour]).
    ``parts`` is the z partition."""

    def __init__(self, rank: int, world: int, parts, wrap: bool, peer_state, peer_flags):
        self.rank, self.world, self.parts = rank, world, parts
        self.lo, self.hi = neighbours(rank, world, wrap)
        self.peer_state, self.peer_flags = peer_state, peer_flags

    def targets(self, k: int, g: int):
        """(put_lo, put_hi, sig_lo, sig_hi) device addresses for writing state k."""
        put_lo = put_hi = sig_lo = sig_hi = 0
        if self.lo is not None:
            t = self.peer_state[k][self.lo]
            n_lo = self.parts[self.lo][1] - self.parts[self.lo][0]
            put_lo = t.data_ptr() + (g + n_lo) * t.stride(0) * 4      # its upper ghost planes
            sig_lo = self.peer_flags[self.lo].data_ptr() + 4          # its "from upper" flag
        if self.hi is not None:
            put_hi = self.peer_state[k][self.hi].data_ptr()           # its lower ghost planes
            sig_hi = self.peer_flags[self.hi].data_ptr()               # its "from lower" flag
        return put_lo, put_hi, sig_lo, sig_hi

    def my_flags(self):
        f = self.peer_flags[self.rank].data_ptr()
        return (f if self.lo is not None else 0), (f + 4 if self.hi is not None else 0)


def fused_step(slab: "SlabPlan", fh: FusedHalo, ins, out: torch.Tensor, out_k: int, value: int, stream) -> None:
    """One time step as ONE kernel launch on ``stream`` (stencil_slab_step_fused):
    the boundary z-chunks run first; before loading ghost planes the kernel
    waits until this rank's flags hold ``value - 1`` (the neighbours' previous
    step); the boundary planes are also stored into the neighbours' ghost
    planes, and each neighbour's flag is raised to ``value`` as soon as the
    chunk it needs is complete."""
    from . import _lib as L
    g = slab.g
    fa, fb = fh.my_flags()
    put_lo, put_hi, sig_lo, sig_hi = fh.targets(out_k, g)
    L.stencil_slab_step_fused(slab.plan.handle, [x.data_ptr() for x in ins], out.data_ptr(), put_lo, put_hi, sig_lo,
                              sig_hi, value, fa, fb, value - 1, int(stream.cuda_stream))


def symmetric_fused_halo(slab: "SlabPlan", group=None):
    """Real multi-GPU setup: two state buffers and the flag array in torch
    symmetric memory (NVLink peer-mapped), rendezvoused over ``group``.
    Returns (state buffers, FusedHalo)."""
    import torch.distributed._symmetric_memory as symm_mem
    grp = group if group is not None else dist.group.WORLD
    dev = torch.device(f"cuda:{slab.plan.device}")
    bufs = [symm_mem.empty(*slab.alloc_shape, dtype=torch.float32, device=dev) for _ in range(2)]
    hdls = [symm_mem.rendezvous(b, grp) for b in bufs]
    flags = symm_mem.empty(2, dtype=torch.int32, device=dev)
    flags.zero_()
    hf = symm_mem.rendezvous(flags, grp)
    torch.cuda.synchronize(dev)
    dist.barrier(group=grp)
    parts = partition(slab.global_extents[0], slab.world)
    peer_state = [[hdls[k].get_buffer(r, slab.alloc_shape, torch.float32) for r in range(slab.world)]
                  for k in range(2)]
    peer_flags = [hf.get_buffer(r, (2,), torch.int32) for r in range(slab.world)]
    return bufs, FusedHalo(slab.rank, slab.world, parts, slab.wrap, peer_state, peer_flags)


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
                         aux_global: Sequence[torch.Tensor] = (), depth: int = 1, time_block: Optional[int] = None,
                         **plan_kw) -> List[torch.Tensor]:
    """Run G slabs on the current device (no process group) and return the
    reassembled global state (newest grid last for ACOUSTIC, else [newest]).
    ``depth`` k > 1: deep halos (r*k ghost planes filled every k steps, the
    overlap recomputed; the schedule of deep_halo_iterate in lockstep)."""
    slabs = [SlabPlan(global_extents, r, world, exchange=_NoExchange(), depth=depth, **plan_kw)
             for r in range(world)]
    if time_block is not None:       # (tests: force two-step passes on grids AUTO keeps single-step)
        for s in slabs:
            s.plan.set_time_block(time_block)
    ex = LocalExchange(slabs)
    nst = len(state_global)
    bufs = [[s.scatter(state_global[k]) if k < nst else s.empty() for k in range(2)] for s in slabs]
    auxs = [[s.scatter(a) for a in aux_global] for s in slabs]
    acoustic = slabs[0].plan.op == 4
    ri = 1 if acoustic else 0
    ex.fill([b[ri] for b in bufs])
    if depth > 1:
        if acoustic:
            ex.fill([b[1 - ri] for b in bufs])
        for k in range(len(aux_global)):
            ex.fill([a[k] for a in auxs])
    # weighted 7-point star with ghosts >= 2: two steps per pass inside the
    # blocks, paired as deep_halo_iterate pairs them (SlabPlan.iterate)
    two = slabs[0].plan.op == 0 and slabs[0].plan.time_block == 2 and slabs[0].r == 1
    t = 0
    while t < n_steps:
        kb = min(depth, n_steps - t)
        j = 1
        while j <= kb:
            dst = 1 - ri
            pair = two and kb >= 2 and (kb % 2 == 0 or j > 1)
            for s, b, a in zip(slabs, bufs, auxs):
                if pair:
                    lo, hi = s.extension((kb - j - 1) * s.r)
                    s.plan.apply2_region(b[ri], out=b[dst], begin=lo, end=hi)
                else:
                    ins = (b[dst], b[ri]) if acoustic else (b[ri],) + tuple(a)
                    lo, hi = s.extension((kb - j) * s.r)
                    s.plan.apply_region(*ins, out=b[dst], begin=lo, end=hi)
            ri = dst
            j += 2 if pair else 1
        ex.fill([b[ri] for b in bufs])
        if acoustic and depth > 1:
            ex.fill([b[1 - ri] for b in bufs])
        t += kb
    out = []
    order = [1 - ri, ri] if acoustic else [ri]
    for k in order:
        out.append(torch.cat([s.owned(b[k]) for s, b in zip(slabs, bufs)], 0))
    return out


class _NoExchange:
    def post(self, buf):
        return []


def virtual_slab_iterate_fused(global_extents, world: int, state_global: Sequence[torch.Tensor], n_steps: int,
                               aux_global: Sequence[torch.Tensor] = (), **plan_kw) -> List[torch.Tensor]:
    """Fused-halo protocol with G slabs in one process: each slab runs on its
    own CUDA stream, the boundary kernels store into the neighbour slabs'
    ghost planes and raise their flags, and the streams synchronise only
    through those flags (stencil_wait_signals) — the multi-GPU protocol with
    device-local "peer" pointers.  A protocol test for grids that do not fill
    the GPU: with every slab's persistent grid on one device, a step t+1 grid
    could occupy every SM while spinning on a flag that a not-yet-resident
    step-t grid must raise; the waits are bounded, so that case ends in a
    StencilError (stencil_device_fault) instead of a hang."""
    slabs = [SlabPlan(global_extents, r, world, exchange=_NoExchange(), **plan_kw) for r in range(world)]
    ex = LocalExchange(slabs)
    nst = len(state_global)
    bufs = [[s.scatter(state_global[k]) if k < nst else s.empty() for k in range(2)] for s in slabs]
    auxs = [[s.scatter(a) for a in aux_global] for s in slabs]
    acoustic = slabs[0].plan.op == 4
    ri = 1 if acoustic else 0
    ex.fill([b[ri] for b in bufs])
    dev = bufs[0][0].device
    flags = [torch.zeros(2, dtype=torch.int32, device=dev) for _ in range(world)]
    parts = partition(global_extents[0], world)
    peer_state = [[bufs[r][k] for r in range(world)] for k in range(2)]
    fhs = [FusedHalo(r, world, parts, slabs[r].wrap, peer_state, flags) for r in range(world)]
    streams = [torch.cuda.Stream(device=dev) for _ in range(world)]
    torch.cuda.synchronize(dev)
    # issue step by step across slabs so no stream waits on work not yet enqueued
    for _ in range(n_steps):
        dst = 1 - ri
        for r, (s, b, a) in enumerate(zip(slabs, bufs, auxs)):
            ins = (b[dst], b[ri]) if acoustic else (b[ri],) + tuple(a)
            s.epoch += 1
            fused_step(s, fhs[r], ins, b[dst], dst, s.epoch, streams[r])
        ri = dst
    torch.cuda.synchronize(dev)
    from . import _lib as L
    L.stencil_device_fault()          # a timed-out flag wait raises here
    order = [1 - ri, ri] if acoustic else [ri]
    return [torch.cat([s.owned(b[k]) for s, b in zip(slabs, bufs)], 0) for k in order]
