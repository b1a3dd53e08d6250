"""Multi-process slab iterate on the GPU: 2-3 ranks (spawned processes) share
cuda:0 and run the real SlabPlan.iterate orchestration (partition, global pad
in z, boundary/interior apply_region split, comm side stream, exchange
pairing incl. the 2-rank ring) with libstencil.so as the compute.  NCCL
refuses two ranks on one device and gloo cannot carry CUDA tensors
point-to-point, so the transport here stages the ghost planes through host
memory over gloo; on a multi-GPU box the same code posts NCCL send/recv.
The gathered result must equal the single-plan iterate bit for bit."""
import os
import socket

import numpy as np
import pytest
import torch
import torch.distributed as dist
import torch.multiprocessing as mp

import stencil_inputs as si

pytestmark = pytest.mark.gpu


def _port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


class StagedExchange:
    """DistExchange's pairing with host-staged buffers (gloo transport)."""

    def __init__(self, rank, world, n, g, wrap, group=None):
        from paper_conf_cgo_hagedornssgd18_b200.slab import DistExchange
        self.inner = DistExchange(rank, world, n, g, wrap, group)

    def post(self, buf):
        ex = self.inner
        n, g = ex.n, ex.g
        if ex.self_wrap or (ex.lo is None and ex.hi is None):
            return ex.post(buf)
        low = buf[g:2 * g].cpu()
        high = buf[n:n + g].cpu()
        rlo, rhi = torch.empty_like(low), torch.empty_like(high)
        ops = []
        if ex.lo is not None:
            ops.append(dist.P2POp(dist.isend, low, ex.lo, tag=0))
        if ex.hi is not None:
            ops.append(dist.P2POp(dist.irecv, rhi, ex.hi, tag=0))
        if ex.hi is not None:
            ops.append(dist.P2POp(dist.isend, high, ex.hi, tag=1))
        if ex.lo is not None:
            ops.append(dist.P2POp(dist.irecv, rlo, ex.lo, tag=1))
        for w in dist.batch_isend_irecv(ops):
            w.wait()
        if ex.lo is not None:
            buf[0:g].copy_(rlo)
        if ex.hi is not None:
            buf[n + g:n + 2 * g].copy_(rhi)
        return []


def _case(name):
    if name == "j3d7_clamp":          # two-step passes (K2R) inside the deep-halo blocks
        ext = (26, 40, 136)
        sp = si.StencilSpec(ext, (3,) * 3, (1,) * 3, (1,) * 3, (1,) * 3, (si.CLAMP,) * 3, 0.0, si.WEIGHTED,
                            si.weights_j3d7(), ())
        return sp, [si.uniform(ext, 94, 0.5, 1.5)], []
    if name == "j3d7_wrap":
        ext = (24, 40, 136)
        sp = si.StencilSpec(ext, (3,) * 3, (1,) * 3, (1,) * 3, (1,) * 3, (si.WRAP,) * 3, 0.0, si.WEIGHTED,
                            si.weights_j3d7(), ())
        return sp, [si.uniform(ext, 90, 0.5, 1.5)], []
    if name == "j3d13_mirror":
        ext = (26, 40, 136)
        sp = si.StencilSpec(ext, (5,) * 3, (1,) * 3, (2,) * 3, (2,) * 3, (si.MIRROR,) * 3, 0.0, si.WEIGHTED,
                            si.weights_j3d13(), ())
        return sp, [si.uniform(ext, 91, 0.5, 1.5)], []
    ext = (24, 36, 132)
    sp = si.StencilSpec(ext, (5,) * 3, (1,) * 3, (2,) * 3, (2,) * 3, (si.CONSTANT,) * 3, 0.0, si.ACOUSTIC, None,
                        si.params_acoustic(13))
    return sp, [si.uniform(ext, 92, -1, 1), si.uniform(ext, 93, -1, 1)], []


def _worker(rank, world, port, name, steps, q, depth=1):
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        torch.cuda.set_device(0)
        import paper_conf_cgo_hagedornssgd18_b200 as lift
        from paper_conf_cgo_hagedornssgd18_b200.slab import SlabPlan
        sp, state, aux = _case(name)
        slab = SlabPlan(sp.extents, rank, world, size=sp.size, pad=sp.pad_lo, kind=list(sp.kind),
                        pad_value=sp.pad_value, op=sp.op, weights=sp.weights, params=sp.params,
                        exchange_factory=StagedExchange, depth=depth)
        if name == "j3d7_clamp":
            slab.plan.set_time_block(2)           # K2R pairs (AUTO keeps single steps on a grid this small)
        bufs = [slab.scatter(torch.from_numpy(x).cuda()) for x in state]
        if len(bufs) == 1:
            bufs.append(slab.empty())
        ri = slab.iterate(bufs, steps)
        torch.cuda.synchronize()
        q.put((rank, slab.owned(bufs[ri]).cpu().numpy()))
        q.put((100 + rank, slab.exchanges))
        if rank == 0:
            plan = lift.Plan.from_spec(sp)
            st = [torch.from_numpy(x).cuda() for x in state]
            if len(st) == 1:
                st.append(torch.empty_like(st[0]))
            rj = plan.iterate(st, steps)
            torch.cuda.synchronize()
            q.put((-1, st[rj].cpu().numpy()))
    finally:
        dist.destroy_process_group()


@pytest.mark.parametrize("name,world,depth", [("j3d7_wrap", 2, 1), ("j3d7_wrap", 3, 1), ("j3d13_mirror", 2, 1),
                                              ("acoustic13", 3, 1), ("j3d7_wrap", 2, 2), ("j3d7_wrap", 3, 4),
                                              ("j3d13_mirror", 2, 2), ("acoustic13", 2, 2), ("j3d7_clamp", 2, 2),
                                              ("j3d7_clamp", 3, 3), ("j3d7_clamp", 2, 4)])
def test_multiprocess_slab_bitwise(name, world, depth):
    """depth k > 1: deep halos (r*k ghost planes every k steps); the number of
    exchanges per rank is ceil(6/k) + 1 (the first fills the initial ghosts)."""
    import __graft_entry__
    __graft_entry__.build()
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _port()
    procs = [ctx.Process(target=_worker, args=(r, world, port, name, 6, q, depth)) for r in range(world)]
    for p in procs:
        p.start()
    res = dict(q.get(timeout=300) for _ in range(2 * world + 1))
    for p in procs:
        p.join(timeout=120)
        assert p.exitcode == 0
    got = np.concatenate([res[r] for r in range(world)], 0)
    np.testing.assert_array_equal(got, res[-1])
    assert all(res[100 + r] == -(-6 // depth) + 1 for r in range(world))
