"""Multi-rank slab decomposition on CPU with gloo.

Each rank owns a z-slab plus ghost planes; the exchange is
paper_conf_cgo_hagedornssgd18_b200.slab.DistExchange (torch.distributed
point-to-point) and the step order is slab.slab_step (boundary planes, then
exchange || interior).  The per-rank compute here is the fp64 oracle on the
rank's local buffer (pad in z only at the global edges), rounded to fp32 per
step, so the decomposed result must equal the oracle's global iterate
(round_fp32=True) bit for bit.  The GPU path runs the same exchange/step code
with libstencil.so as the compute.
"""
import os
import socket

import numpy as np
import pytest
import torch
import torch.distributed as dist
import torch.multiprocessing as mp

import stencil_inputs as si
from oracle import stencil_oracle as orc
from paper_conf_cgo_hagedornssgd18_b200.slab import DistExchange, neighbours, partition, slab_step


def _free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def _spec(extents, kind, size=3, weights=None):
    w = si.weights_j3d7() if size == 3 else si.weights_j3d13()
    r = size // 2
    return si.StencilSpec(tuple(extents), (size,) * 3, (1, 1, 1), (r,) * 3, (r,) * 3, (kind,) * 3, 0.25,
                          si.WEIGHTED, w, ())


def _local_compute(spec, gext, rank, world, z0, n, g, inp, out, a, b):
    """Owned output planes [a, b) of the slab from its ghost-extended buffer."""
    wrap = spec.kind[0] == si.WRAP
    lo = spec.pad_lo[0]
    first = rank == 0 and not wrap
    last = rank == world - 1 and not wrap
    x = inp.numpy().astype(np.float64)
    zlo = g if first else g - lo            # first input plane used
    zhi = g + n if last else g + n + lo     # one past the last
    sub = x[zlo:zhi]
    sp = si.StencilSpec((zhi - zlo,) + tuple(gext[1:]), spec.size, spec.step,
                        (lo if first else 0,) + spec.pad_lo[1:], (lo if last else 0,) + spec.pad_hi[1:],
                        spec.kind, spec.pad_value, spec.op, spec.weights, spec.params)
    Y, _ = orc.apply(sp, [sub])
    assert Y.shape[0] == n
    out[g + a:g + b] = torch.from_numpy(Y[a:b].astype(np.float32))


def _worker(rank, world, port, kind, size, steps, q):
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        gext = (11, 6, 8)
        spec = _spec(gext, kind, size)
        g = size // 2
        z0, z1 = partition(gext[0], world)[rank]
        n = z1 - z0
        xg = si.uniform(gext, 2024, 0.5, 1.5)
        bufs = [torch.zeros((n + 2 * g,) + gext[1:]), torch.zeros((n + 2 * g,) + gext[1:])]
        bufs[0][g:g + n] = torch.from_numpy(xg[z0:z1])
        ex = DistExchange(rank, world, n, g, kind == si.WRAP)
        for w in ex.post(bufs[0]):
            w.wait()
        cur = 0
        for _ in range(steps):
            inp, out = bufs[cur], bufs[1 - cur]
            works = slab_step(lambda a, b: _local_compute(spec, gext, rank, world, z0, n, g, inp, out, a, b),
                              lambda: ex.post(out), n, g)
            for w in works:
                w.wait()
            cur = 1 - cur
        q.put((rank, z0, bufs[cur][g:g + n].numpy().copy(), bufs[cur].numpy().copy()))
    finally:
        dist.destroy_process_group()


def _run(world, kind, size=3, steps=3):
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _free_port()
    procs = [ctx.Process(target=_worker, args=(r, world, port, kind, size, steps, q)) for r in range(world)]
    for p in procs:
        p.start()
    res = [q.get(timeout=240) for _ in range(world)]
    for p in procs:
        p.join(timeout=60)
        assert p.exitcode == 0
    res.sort()
    return res


def test_partition_and_neighbours():
    assert partition(10, 3) == [(0, 3), (3, 6), (6, 10)]
    assert partition(512 * 8, 8)[7] == (7 * 512, 8 * 512)
    with pytest.raises(ValueError):
        partition(2, 3)
    assert neighbours(0, 4, False) == (None, 1)
    assert neighbours(3, 4, False) == (2, None)
    assert neighbours(0, 4, True) == (3, 1)
    assert neighbours(1, 2, True) == (0, 0)


@pytest.mark.parametrize("world", [2, 3])
@pytest.mark.parametrize("kind", [si.CLAMP, si.WRAP, si.CONSTANT, si.MIRROR])
def test_gloo_slab_iterate_matches_global_oracle(world, kind):
    steps = 3
    res = _run(world, kind, 3, steps)
    got = np.concatenate([r[2] for r in res], 0)
    gext = (11, 6, 8)
    ref = orc.iterate(_spec(gext, kind), [si.uniform(gext, 2024, 0.5, 1.5)], [], steps, round_fp32=True)[0]
    np.testing.assert_array_equal(got, ref.astype(np.float32))


def test_gloo_slab_radius2_ghosts():
    res = _run(2, si.REFLECT, 5, 2)
    got = np.concatenate([r[2] for r in res], 0)
    gext = (11, 6, 8)
    ref = orc.iterate(_spec(gext, si.REFLECT, 5), [si.uniform(gext, 2024, 0.5, 1.5)], [], 2, round_fp32=True)[0]
    np.testing.assert_array_equal(got, ref.astype(np.float32))


# ------------------------------------------------ deep halos (NEXT-3) -------
def _region_compute(spec, gext, rank, world, n, g, inp, out, a, b):
    """Output planes [a, b) (slab-local; a < 0 / b > n reach into the ghosts)
    from the ghost-extended buffer ``inp`` with the fp64 oracle; pad in z only
    at a global, non-periodic edge."""
    wrap = spec.kind[0] == si.WRAP
    lo, hi = spec.pad_lo[0], spec.pad_hi[0]
    first = rank == 0 and not wrap and a == 0
    last = rank == world - 1 and not wrap and b == n
    x = inp.numpy().astype(np.float64)
    zlo = g + a if first else g + a - lo
    zhi = g + b if last else g + b + hi
    assert zlo >= 0 and zhi <= n + 2 * g, "region reads outside the ghost planes"
    sp = si.StencilSpec((zhi - zlo,) + tuple(gext[1:]), spec.size, spec.step,
                        (lo if first else 0,) + spec.pad_lo[1:], (hi if last else 0,) + spec.pad_hi[1:],
                        spec.kind, spec.pad_value, spec.op, spec.weights, spec.params)
    Y, _ = orc.apply(sp, [x[zlo:zhi]])
    assert Y.shape[0] == b - a
    out[g + a:g + b] = torch.from_numpy(Y.astype(np.float32))


def _deep_worker(rank, world, port, kind, size, steps, depth, q, two=False):
    from paper_conf_cgo_hagedornssgd18_b200.slab import deep_halo_iterate
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        gext = (23, 6, 8)
        spec = _spec(gext, kind, size)
        r = size // 2
        g = r * depth
        z0, z1 = partition(gext[0], world)[rank]
        n = z1 - z0
        wrap = kind == si.WRAP
        xg = si.uniform(gext, 2025, 0.5, 1.5)
        bufs = [torch.zeros((n + 2 * g,) + gext[1:]), torch.zeros((n + 2 * g,) + gext[1:])]
        bufs[0][g:g + n] = torch.from_numpy(xg[z0:z1])
        ex = DistExchange(rank, world, n, g, wrap)
        lo_nb, hi_nb = neighbours(rank, world, wrap)
        posts = []

        def extension(e):
            return (-e if lo_nb is not None else 0), (n + e if hi_nb is not None else n)

        def compute(src, dst, a, b):
            _region_compute(spec, gext, rank, world, n, g, bufs[src], bufs[dst], a, b)

        def post(grids):
            posts.append(len(grids))
            works = []
            for i in grids:
                works += ex.post(bufs[i])
            return works

        def join(works):
            for w in works:
                w.wait()

        def compute2(src, dst, a, b):
            # two steps over [a, b): the first over the region widened by r,
            # except at a global non-periodic edge (there the intermediate grid
            # is padded instead), as stencil_apply2_region does
            tmp = torch.zeros_like(bufs[0])
            a1 = a if (a == 0 and lo_nb is None) else a - r
            b1 = b if (b == n and hi_nb is None) else b + r
            _region_compute(spec, gext, rank, world, n, g, bufs[src], tmp, a1, b1)
            _region_compute(spec, gext, rank, world, n, g, tmp, bufs[dst], a, b)

        ri = deep_halo_iterate(steps, depth, r, n, g, extension, compute, post, lambda f: f(), join, False, 0,
                               compute2=compute2 if two else None)
        q.put((rank, z0, bufs[ri][g:g + n].numpy().copy(), len(posts)))
    finally:
        dist.destroy_process_group()


@pytest.mark.parametrize("depth", [2, 4])
@pytest.mark.parametrize("world,kind,size", [(2, si.CLAMP, 3), (3, si.WRAP, 3), (2, si.MIRROR, 5),
                                             (3, si.CONSTANT, 3)])
def test_gloo_deep_halo_matches_global_oracle(world, kind, size, depth):
    """Ghosts of r*k planes exchanged every k steps, the overlap recomputed:
    bit-for-bit the oracle's global iterate (fp32 rounding per step), with
    ceil(steps/k) + 1 exchanges (the first fills the initial ghosts)."""
    steps = 7
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _free_port()
    procs = [ctx.Process(target=_deep_worker, args=(r, world, port, kind, size, steps, depth, q))
             for r in range(world)]
    for p in procs:
        p.start()
    res = sorted(q.get(timeout=240) for _ in range(world))
    for p in procs:
        p.join(timeout=60)
        assert p.exitcode == 0
    got = np.concatenate([r[2] for r in res], 0)
    gext = (23, 6, 8)
    ref = orc.iterate(_spec(gext, kind, size), [si.uniform(gext, 2025, 0.5, 1.5)], [], steps, round_fp32=True)[0]
    np.testing.assert_array_equal(got, ref.astype(np.float32))
    assert all(r[3] == -(-steps // depth) + 1 for r in res)


@pytest.mark.parametrize("depth", [2, 3, 4])
@pytest.mark.parametrize("world,kind,size", [(2, si.CLAMP, 3), (3, si.WRAP, 3), (2, si.MIRROR, 5)])
def test_gloo_deep_halo_two_step_pairs_match_global_oracle(world, kind, size, depth):
    """The deep-halo schedule with two-step passes (compute2: the pairing used
    with stencil_apply2_region on the GPU — pairs of steps over the second
    step's region, an odd block starting with one single step, the block's
    last pair split into boundary / exchange || interior): bit-for-bit the
    oracle's global iterate, same exchange count."""
    steps = 7
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _free_port()
    procs = [ctx.Process(target=_deep_worker, args=(r, world, port, kind, size, steps, depth, q, True))
             for r in range(world)]
    for p in procs:
        p.start()
    res = sorted(q.get(timeout=240) for _ in range(world))
    for p in procs:
        p.join(timeout=60)
        assert p.exitcode == 0
    got = np.concatenate([r[2] for r in res], 0)
    gext = (23, 6, 8)
    ref = orc.iterate(_spec(gext, kind, size), [si.uniform(gext, 2025, 0.5, 1.5)], [], steps, round_fp32=True)[0]
    np.testing.assert_array_equal(got, ref.astype(np.float32))
    assert all(r[3] == -(-steps // depth) + 1 for r in res)
