"""Scheduling independence of the persistent kernels and bounded halo waits.

Results must not depend on how launches are scheduled (tiling and parallel
execution preserve the stencil's semantics):

  * the persistent kernels' work counters belong to one launch at a time
    (slots.cuh): two CUDA graphs replayed CONCURRENTLY on two streams —
    including graphs captured 4096 launches apart, which shared a counter slot
    under the round-1 host-side slot ring — give bitwise the single-stream
    result, for K2 (3D sweep), K3 (2D per-warp sweeps) and K1S;
  * a fused-halo wait whose neighbour never raises its flag (a dead rank)
    times out and is reported as STENCIL_E_CUDA instead of hanging the GPU.
"""
import numpy as np
import pytest
import torch

import stencil_inputs as si

pytestmark = pytest.mark.gpu


@pytest.fixture(scope="module")
def lift():
    import __graft_entry__
    __graft_entry__.build()
    import paper_conf_cgo_hagedornssgd18_b200 as m
    torch.cuda.set_device(0)
    return m


def _graph(fn, stream):
    g = torch.cuda.CUDAGraph()
    with torch.cuda.stream(stream):
        fn()                                  # warm-up (TMA descriptors cached)
        torch.cuda.current_stream().synchronize()
        with torch.cuda.graph(g, stream=stream):
            fn()
    return g


CASES = {
    # (extents, spec builder, variant the plan must run on)
    "k2_j3d7": ((96, 256, 512), lambda e: si.StencilSpec(e, (3,) * 3, (1,) * 3, (1,) * 3, (1,) * 3,
                                                          (si.CLAMP,) * 3, 0.0, si.WEIGHTED, si.weights_j3d7(), ()),
                2),
    "k3_j2d9": ((2048, 2048), lambda e: si.StencilSpec(e, (3, 3), (1, 1), (1, 1), (1, 1), (si.CLAMP,) * 2, 0.0,
                                                        si.WEIGHTED, si.weights_j2d9(), ()), 1),
    "k1s_srad": ((1024, 1024), lambda e: si.StencilSpec(e, (3, 3), (1, 1), (1, 1), (1, 1), (si.CLAMP,) * 2, 0.0,
                                                         si.SRAD, None, si.params_srad2()), 1),
}


@pytest.mark.parametrize("case", list(CASES))
@pytest.mark.parametrize("gap", [0, 4096])
def test_concurrent_graph_replay_bitwise(lift, case, gap):
    """Graph A (plan P, 3 steps) is captured; then ``gap`` unrelated launches
    of another persistent-kernel plan; then graph B (a second plan of the same
    problem, 3 steps).  A and B are replayed 8 times at once on two streams;
    every replay must give exactly the eager single-stream result."""
    ext, mk, var = CASES[case]
    sp = mk(ext)
    x = (np.exp(si.uniform(ext, 91, 0.0, 1.0)) if sp.op == si.SRAD else si.uniform(ext, 91, 0.5, 1.5)).astype(np.float32)
    pa, pb = lift.Plan.from_spec(sp), lift.Plan.from_spec(sp)
    xa, xb = torch.from_numpy(x).cuda(), torch.from_numpy(x).cuda()
    ya, yb = torch.empty_like(xa), torch.empty_like(xb)
    # reference: eager, one stream
    ref_in, ref_out = torch.from_numpy(x).cuda(), torch.empty_like(xa)
    ri = pa.iterate([ref_in, ref_out], 3)
    torch.cuda.synchronize()
    ref = (ref_in, ref_out)[ri].cpu().numpy()
    assert pa.last_variant == var
    sa, sb = torch.cuda.Stream(), torch.cuda.Stream()
    xa0, xb0 = xa.clone(), xb.clone()
    ga = _graph(lambda: pa.iterate([xa, ya], 3), sa)
    if gap:
        small = lift.Plan.from_spec(si.StencilSpec((16, 16, 64), (3,) * 3, (1,) * 3, (1,) * 3, (1,) * 3,
                                                   (si.CLAMP,) * 3, 0.0, si.WEIGHTED, si.weights_j3d7(), ()))
        u = torch.rand(16, 16, 64, device="cuda")
        v = torch.empty_like(u)
        for _ in range(gap):
            small.apply(u, out=v)
        torch.cuda.synchronize()
    gb = _graph(lambda: pb.iterate([xb, yb], 3), sb)
    for rep in range(8):
        xa.copy_(xa0)
        xb.copy_(xb0)
        torch.cuda.synchronize()
        with torch.cuda.stream(sa):
            ga.replay()
        with torch.cuda.stream(sb):
            gb.replay()
        torch.cuda.synchronize()
        # iterate with 3 steps ends in the second buffer (odd step count)
        np.testing.assert_array_equal((xa, ya)[ri].cpu().numpy(), ref, err_msg=f"graph A, replay {rep}")
        np.testing.assert_array_equal((xb, yb)[ri].cpu().numpy(), ref, err_msg=f"graph B, replay {rep}")


def test_concurrent_eager_plans_on_streams(lift):
    """Eight launches of two plans interleaved on two streams (no graphs)."""
    ext = (64, 256, 512)
    sp = CASES["k2_j3d7"][1](ext)
    x = si.uniform(ext, 92, 0.5, 1.5)
    plan = lift.Plan.from_spec(sp)
    xs = [torch.from_numpy(x).cuda() for _ in range(4)]
    ys = [torch.empty_like(xs[0]) for _ in range(4)]
    streams = [torch.cuda.Stream() for _ in range(4)]
    torch.cuda.synchronize()
    for k in range(4):
        plan.apply(xs[k], out=ys[k], stream=streams[k])
    torch.cuda.synchronize()
    plan.apply(xs[0], out=ys[0])
    torch.cuda.synchronize()
    ref = ys[0].cpu().numpy()
    for k in range(1, 4):
        np.testing.assert_array_equal(ys[k].cpu().numpy(), ref)


@pytest.fixture
def short_timeout(lift):
    lift.stencil_set_wait_timeout_ms(300)
    yield
    lift.stencil_set_wait_timeout_ms(10000)


def test_wait_signals_dead_neighbour_times_out(lift, short_timeout):
    from paper_conf_cgo_hagedornssgd18_b200 import StencilError
    flags = torch.zeros(2, dtype=torch.int32, device="cuda")
    lift.stencil_device_fault()                       # nothing pending
    lift.stencil_wait_signals(flags.data_ptr(), 0, 7, torch.cuda.current_stream().cuda_stream)
    torch.cuda.synchronize()                          # returns: the wait gave up
    with pytest.raises(StencilError, match="lower neighbour never raised"):
        lift.stencil_device_fault()
    lift.stencil_device_fault()                       # cleared by the check
    # a raised flag passes without a fault
    flags.fill_(7)
    lift.stencil_wait_signals(flags.data_ptr(), flags.data_ptr() + 4, 7, torch.cuda.current_stream().cuda_stream)
    torch.cuda.synchronize()
    lift.stencil_device_fault()


def test_fused_step_dead_neighbour_returns_e_cuda(lift, short_timeout):
    """A fused slab step waiting on an upper neighbour that never signals
    finishes (stale ghosts) instead of hanging; the fault is reported by the
    next fused call and by stencil_device_fault; the GPU stays usable."""
    from paper_conf_cgo_hagedornssgd18_b200 import StencilError
    from paper_conf_cgo_hagedornssgd18_b200.slab import SlabPlan, _NoExchange
    ext = (64, 64, 128)
    s = SlabPlan(ext, 0, 2, size=3, kind="clamp", weights=si.weights_j3d7(), exchange=_NoExchange())
    a, b = s.empty().normal_(), s.empty()
    flags = torch.zeros(2, dtype=torch.int32, device="cuda")
    st = torch.cuda.current_stream().cuda_stream
    lift.stencil_slab_step_fused(s.plan.handle, [a.data_ptr()], b.data_ptr(), 0, 0, 0, 0, 1, 0,
                                 flags.data_ptr() + 4, 5, st)
    torch.cuda.synchronize()
    with pytest.raises(StencilError, match="upper neighbour never raised"):
        lift.stencil_slab_step_fused(s.plan.handle, [a.data_ptr()], b.data_ptr(), 0, 0, 0, 0, 1, 0,
                                     flags.data_ptr() + 4, 5, st)
    # the device is healthy: a normal launch still runs and is correct
    flags.fill_(5)
    lift.stencil_slab_step_fused(s.plan.handle, [a.data_ptr()], b.data_ptr(), 0, 0, 0, 0, 1, 0,
                                 flags.data_ptr() + 4, 5, st)
    torch.cuda.synchronize()
    lift.stencil_device_fault()
