"""Slab decomposition on the GPU (single device): the decomposed iterate must be
bitwise equal to the single-plan iterate (same per-point kernel code), and the
single-plan iterate matches the oracle (test_parity_gpu).

  * virtual slabs: G slab plans on one device, ghosts filled by D2D copies
    (slab.virtual_slab_iterate) — checks partition, ghost layout, global pad
    handling in z (stencil_plan_set_slab) and the Acoustic global neighbour
    count;
  * SlabPlan with world = 1: the boundary / interior apply_region split, the
    comm side stream and the exchange hook of the multi-GPU path.
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


def single_iterate(lift, spec, state, aux, n):
    plan = lift.Plan.from_spec(spec)
    st = [torch.from_numpy(x).cuda() for x in state]
    if len(st) == 1:
        st.append(torch.empty_like(st[0]))
    ax = [torch.from_numpy(x).cuda() for x in aux]
    ri = plan.iterate(st, n, ax)
    torch.cuda.synchronize()
    if spec.op == si.ACOUSTIC:
        return [st[1 - ri].cpu().numpy(), st[ri].cpu().numpy()]
    return [st[ri].cpu().numpy()]


def kw(spec):
    return dict(size=spec.size, pad=spec.pad_lo, kind=list(spec.kind), pad_value=spec.pad_value, op=spec.op,
                weights=spec.weights, params=spec.params)


@pytest.mark.parametrize("kind", [si.CLAMP, si.WRAP, si.CONSTANT, si.MIRROR, si.REFLECT])
@pytest.mark.parametrize("world", [2, 3])
def test_virtual_slab_weighted_bitwise(lift, kind, world):
    from paper_conf_cgo_hagedornssgd18_b200.slab import virtual_slab_iterate
    ext = (30, 40, 136)
    sp = si.StencilSpec(ext, (3,) * 3, (1,) * 3, (1,) * 3, (1,) * 3, (kind,) * 3, 0.5, si.WEIGHTED,
                        si.weights_j3d7(), ())
    x = si.uniform(ext, 77, 0.5, 1.5)
    ref = single_iterate(lift, sp, [x], [], 5)[0]
    got = virtual_slab_iterate(ext, world, [torch.from_numpy(x).cuda()], 5, **kw(sp))[0]
    np.testing.assert_array_equal(got.cpu().numpy(), ref)


@pytest.mark.parametrize("kind", [si.CLAMP, si.WRAP, si.CONSTANT])
def test_virtual_slab_gather_bitwise(lift, kind):
    """Slabs on the K5 gather kernel (nx % 4 != 0 rules out TMA; a 5x5x5 box):
    ghost planes, global-z pad and output regions as in the single plan."""
    from paper_conf_cgo_hagedornssgd18_b200.slab import virtual_slab_iterate
    ext = (26, 20, 66)
    w = np.random.default_rng(96).standard_normal((5, 5, 5)).astype(np.float32) * 0.01
    sp = si.StencilSpec(ext, (5,) * 3, (1,) * 3, (2,) * 3, (2,) * 3, (kind,) * 3, 0.25, si.WEIGHTED, w, ())
    assert lift.Plan.from_spec(sp).variant == lift.plan.VARIANTS["gather"]
    x = si.uniform(ext, 97, 0.5, 1.5)
    ref = single_iterate(lift, sp, [x], [], 3)[0]
    got = virtual_slab_iterate(ext, 3, [torch.from_numpy(x).cuda()], 3, **kw(sp))[0]
    np.testing.assert_array_equal(got.cpu().numpy(), ref)


@pytest.mark.parametrize("pts,sz", [(7, 3), (13, 5)])
def test_virtual_slab_acoustic_bitwise(lift, pts, sz):
    from paper_conf_cgo_hagedornssgd18_b200.slab import virtual_slab_iterate
    ext = (24, 36, 132)
    r = sz // 2
    sp = si.StencilSpec(ext, (sz,) * 3, (1,) * 3, (r,) * 3, (r,) * 3, (si.CONSTANT,) * 3, 0.0, si.ACOUSTIC, None,
                        si.params_acoustic(pts))
    u0 = si.uniform(ext, 78, -1, 1)
    u1 = si.uniform(ext, 79, -1, 1)
    ref = single_iterate(lift, sp, [u0, u1], [], 4)
    got = virtual_slab_iterate(ext, 3, [torch.from_numpy(u0).cuda(), torch.from_numpy(u1).cuda()], 4, **kw(sp))
    np.testing.assert_array_equal(got[1].cpu().numpy(), ref[1])
    np.testing.assert_array_equal(got[0].cpu().numpy(), ref[0])


def test_virtual_slab_hotspot_bitwise(lift):
    from paper_conf_cgo_hagedornssgd18_b200.slab import virtual_slab_iterate
    ext = (8, 64, 128)
    sp = si.StencilSpec(ext, (3,) * 3, (1,) * 3, (1,) * 3, (1,) * 3, (si.CLAMP,) * 3, 0.0, si.HOTSPOT3D, None,
                        si.params_hotspot3d())
    T = si.uniform(ext, 80, 300, 350)
    P = si.uniform(ext, 81, 0, 1e-2)
    ref = single_iterate(lift, sp, [T], [P], 6)[0]
    got = virtual_slab_iterate(ext, 2, [torch.from_numpy(T).cuda()], 6, [torch.from_numpy(P).cuda()], **kw(sp))[0]
    np.testing.assert_array_equal(got.cpu().numpy(), ref)


@pytest.mark.parametrize("kind", [si.CLAMP, si.WRAP])
def test_slabplan_world1_split_bitwise(lift, kind):
    from paper_conf_cgo_hagedornssgd18_b200.slab import SlabPlan
    ext = (20, 40, 136)
    sp = si.StencilSpec(ext, (3,) * 3, (1,) * 3, (1,) * 3, (1,) * 3, (kind,) * 3, 0.0, si.WEIGHTED,
                        si.weights_j3d7(), ())
    x = si.uniform(ext, 82, 0.5, 1.5)
    ref = single_iterate(lift, sp, [x], [], 7)[0]
    slab = SlabPlan(ext, 0, 1, **kw(sp))
    a = slab.scatter(torch.from_numpy(x).cuda())
    b = slab.empty()
    ri = slab.iterate([a, b], 7)
    torch.cuda.synchronize()
    np.testing.assert_array_equal(slab.owned((a, b)[ri]).cpu().numpy(), ref)


@pytest.mark.parametrize("kind,world", [(si.CLAMP, 2), (si.CLAMP, 3), (si.WRAP, 2), (si.WRAP, 3), (si.WRAP, 1),
                                        (si.MIRROR, 4)])
def test_fused_halo_virtual_bitwise(lift, kind, world):
    """Fused halo put: boundary kernels store into the neighbour slabs' ghosts
    and raise their flags; each slab on its own stream, synchronised only by
    the flags — bitwise equal to the single plan."""
    from paper_conf_cgo_hagedornssgd18_b200.slab import virtual_slab_iterate_fused
    ext = (32, 40, 136)
    sp = si.StencilSpec(ext, (3,) * 3, (1,) * 3, (1,) * 3, (1,) * 3, (kind,) * 3, 0.0, si.WEIGHTED,
                        si.weights_j3d7(), ())
    x = si.uniform(ext, 83, 0.5, 1.5)
    ref = single_iterate(lift, sp, [x], [], 9)[0]
    got = virtual_slab_iterate_fused(ext, world, [torch.from_numpy(x).cuda()], 9, **kw(sp))[0]
    np.testing.assert_array_equal(got.cpu().numpy(), ref)


def test_fused_halo_virtual_acoustic13(lift):
    from paper_conf_cgo_hagedornssgd18_b200.slab import virtual_slab_iterate_fused
    ext = (30, 36, 132)
    sp = si.StencilSpec(ext, (5,) * 3, (1,) * 3, (2,) * 3, (2,) * 3, (si.CONSTANT,) * 3, 0.0, si.ACOUSTIC, None,
                        si.params_acoustic(13))
    u0 = si.uniform(ext, 84, -1, 1)
    u1 = si.uniform(ext, 85, -1, 1)
    ref = single_iterate(lift, sp, [u0, u1], [], 6)
    got = virtual_slab_iterate_fused(ext, 3, [torch.from_numpy(u0).cuda(), torch.from_numpy(u1).cuda()], 6,
                                     **kw(sp))
    np.testing.assert_array_equal(got[1].cpu().numpy(), ref[1])
    np.testing.assert_array_equal(got[0].cpu().numpy(), ref[0])


def test_apply_region_put_needs_slab(lift):
    sp = si.StencilSpec((16, 40, 136), (3,) * 3, (1,) * 3, (1,) * 3, (1,) * 3, (si.CLAMP,) * 3, 0.0, si.WEIGHTED,
                        si.weights_j3d7(), ())
    plan = lift.Plan.from_spec(sp)
    x = torch.zeros(sp.extents, device="cuda")
    y = torch.empty_like(x)
    with pytest.raises(lift.StencilError) as e:
        lift.stencil_apply_region_put(plan.handle, [x.data_ptr()], y.data_ptr(), 0, 1)
    assert e.value.status == 1


# ------------------------------------------------ deep halos (NEXT-3) -------
DEEP_CASES = {
    "j3d7_clamp": lambda: (si.StencilSpec((40, 40, 136), (3,) * 3, (1,) * 3, (1,) * 3, (1,) * 3, (si.CLAMP,) * 3,
                                          0.0, si.WEIGHTED, si.weights_j3d7(), ()), [si.uniform((40, 40, 136), 95)],
                           []),
    "j3d7_wrap": lambda: (si.StencilSpec((40, 40, 136), (3,) * 3, (1,) * 3, (1,) * 3, (1,) * 3, (si.WRAP,) * 3,
                                         0.0, si.WEIGHTED, si.weights_j3d7(), ()), [si.uniform((40, 40, 136), 96)],
                          []),
    "j3d13_mirror": lambda: (si.StencilSpec((48, 40, 136), (5,) * 3, (1,) * 3, (2,) * 3, (2,) * 3,
                                            (si.MIRROR,) * 3, 0.0, si.WEIGHTED, si.weights_j3d13(), ()),
                             [si.uniform((48, 40, 136), 97)], []),
    "acoustic13": lambda: (si.StencilSpec((48, 36, 132), (5,) * 3, (1,) * 3, (2,) * 3, (2,) * 3,
                                          (si.CONSTANT,) * 3, 0.0, si.ACOUSTIC, None, si.params_acoustic(13)),
                           [si.uniform((48, 36, 132), 98, -1, 1), si.uniform((48, 36, 132), 99, -1, 1)], []),
    # a 5x5x5 box (K5 gather tiles) and an odd-width 3x3x3 box (K0 rows / K5):
    # the regions reaching into the ghosts on the non-TMA kernel families
    "box5_k5": lambda: (si.StencilSpec((48, 20, 36), (5,) * 3, (1,) * 3, (2,) * 3, (2,) * 3, (si.REFLECT,) * 3, 0.0,
                                       si.WEIGHTED, (np.random.default_rng(5).random((5, 5, 5)) / 125).astype(np.float32),
                                       ()), [si.uniform((48, 20, 36), 102)], []),
    "box3_odd_width": lambda: (si.StencilSpec((40, 24, 37), (3,) * 3, (1,) * 3, (1,) * 3, (1,) * 3, (si.WRAP,) * 3, 0.0,
                                              si.WEIGHTED, (np.random.default_rng(6).random((3, 3, 3)) / 27).astype(
                                                  np.float32), ()), [si.uniform((40, 24, 37), 103)], []),
    # Acoustic on an odd width runs on K0 (one thread per output)
    "acoustic7_k0": lambda: (si.StencilSpec((40, 20, 37), (3,) * 3, (1,) * 3, (1,) * 3, (1,) * 3, (si.CONSTANT,) * 3,
                                            0.0, si.ACOUSTIC, None, si.params_acoustic(7)),
                             [si.uniform((40, 20, 37), 104, -1, 1), si.uniform((40, 20, 37), 105, -1, 1)], []),
    "hotspot3d": lambda: (si.StencilSpec((40, 64, 128), (3,) * 3, (1,) * 3, (1,) * 3, (1,) * 3, (si.CLAMP,) * 3,
                                         0.0, si.HOTSPOT3D, None, si.params_hotspot3d()),
                          [si.uniform((40, 64, 128), 100, 300, 350)], [si.uniform((40, 64, 128), 101, 0, 0.01)]),
}


@pytest.mark.parametrize("depth", [2, 3, 4])
@pytest.mark.parametrize("world", [1, 2, 3])
@pytest.mark.parametrize("case", list(DEEP_CASES))
def test_virtual_slab_deep_halo_bitwise(lift, case, world, depth):
    """Deep halos: ghosts of r*k planes filled every k steps, the overlap of
    the extended regions recomputed by apply_region into the ghost planes —
    bitwise equal to the single-plan iterate (7 steps: a partial last block)."""
    from paper_conf_cgo_hagedornssgd18_b200.slab import virtual_slab_iterate
    sp, state, aux = DEEP_CASES[case]()
    ref = single_iterate(lift, sp, state, aux, 7)
    tb = 2 if case == "j3d7_clamp" else None     # (K2R pairs inside the blocks; AUTO skips grids this small)
    got = virtual_slab_iterate(sp.extents, world, [torch.from_numpy(x).cuda() for x in state], 7,
                               [torch.from_numpy(x).cuda() for x in aux], depth=depth, time_block=tb, **kw(sp))
    for g_, r_ in zip(got, ref):
        np.testing.assert_array_equal(g_.cpu().numpy(), r_)


def test_apply_region_into_ghosts_validation(lift):
    """A slab plan's region may reach ghost - pad planes into the ghosts, no
    further; an unslabbed plan may not leave [0, n)."""
    from paper_conf_cgo_hagedornssgd18_b200 import StencilError
    from paper_conf_cgo_hagedornssgd18_b200.slab import SlabPlan, _NoExchange
    s = SlabPlan((40, 40, 136), 1, 3, size=3, kind="clamp", weights=si.weights_j3d7(), exchange=_NoExchange(),
                 depth=4)
    a, b = s.empty().uniform_(), s.empty()
    s.plan.apply_region(a, out=b, begin=-3, end=s.n + 3)
    with pytest.raises(StencilError):
        s.plan.apply_region(a, out=b, begin=-4, end=s.n)
    with pytest.raises(StencilError):
        s.plan.apply_region(a, out=b, begin=0, end=s.n + 4)


# ------------------------------ two steps per pass inside deep-halo blocks ---
def _j3d7(ext, kind):
    return si.StencilSpec(tuple(ext), (3,) * 3, (1,) * 3, (1,) * 3, (1,) * 3, (kind,) * 3, 0.0, si.WEIGHTED,
                          si.weights_j3d7(), ())


def test_apply2_region_bitwise_and_limits(lift):
    """stencil_apply2_region = two apply_region steps (the first over the
    region widened by the pad) on an unslabbed plan and on a slab reaching into
    its ghosts; limits and errors."""
    from paper_conf_cgo_hagedornssgd18_b200 import StencilError
    from paper_conf_cgo_hagedornssgd18_b200.slab import SlabPlan, _NoExchange
    sp = _j3d7((40, 40, 136), si.CLAMP)
    plan = lift.Plan.from_spec(sp)
    x = torch.from_numpy(si.uniform((40, 40, 136), 120, 0.5, 1.5)).cuda()
    ref1, ref2 = torch.zeros_like(x), torch.zeros_like(x)
    plan.apply_region(x, out=ref1, begin=4, end=31)
    plan.apply_region(ref1, out=ref2, begin=5, end=30)
    got = torch.zeros_like(x)
    plan.apply2_region(x, out=got, begin=5, end=30)
    assert plan.last_kernel == "k2r_sweep"
    assert torch.equal(got[5:30], ref2[5:30])
    with pytest.raises(StencilError):
        plan.apply2_region(x, out=x, begin=0, end=40)              # aliasing
    with pytest.raises(StencilError):
        plan.apply2_region(x, out=got, begin=-1, end=40)           # unslabbed: [0, n) only
    wrap = lift.Plan.from_spec(_j3d7((40, 40, 136), si.WRAP))
    with pytest.raises(StencilError):
        wrap.apply2_region(x, out=got, begin=0, end=40)            # no two-step kernel
    s = SlabPlan((40, 40, 136), 1, 3, size=3, kind="clamp", weights=si.weights_j3d7(), exchange=_NoExchange(),
                 depth=4)
    a, b1, b2, c = s.empty().uniform_(), s.empty().zero_(), s.empty().zero_(), s.empty().zero_()
    s.plan.apply_region(a, out=b1, begin=-3, end=s.n + 3)
    s.plan.apply_region(b1, out=b2, begin=-2, end=s.n + 2)
    s.plan.apply2_region(a, out=c, begin=-2, end=s.n + 2)
    g = s.g
    assert torch.equal(c[g - 2:g + s.n + 2], b2[g - 2:g + s.n + 2])
    with pytest.raises(StencilError):
        s.plan.apply2_region(a, out=c, begin=-3, end=s.n)          # ghost - 2 pads = 2


def test_slabplan_two_step_blocks(lift):
    """SlabPlan.iterate (world 1, depth 4 and 3) runs the weighted 7-point
    blocks as two-step passes (K2R) and gives the single-plan bits."""
    from paper_conf_cgo_hagedornssgd18_b200.slab import SlabPlan, _NoExchange
    x = si.uniform((40, 40, 136), 121, 0.5, 1.5)
    sp = _j3d7(x.shape, si.CLAMP)
    for depth, n in ((4, 8), (3, 9)):            # blocks end with a two-step pair
        ref = single_iterate(lift, sp, [x], [], n)[0]
        s = SlabPlan(x.shape, 0, 1, size=3, kind="clamp", weights=si.weights_j3d7(), exchange=_NoExchange(),
                     depth=depth)
        s.plan.set_time_block(2)                 # (AUTO keeps single steps on a grid this small)
        a, b = s.scatter(torch.from_numpy(x).cuda()), s.empty()
        ri = s.iterate([a, b], n)
        torch.cuda.synchronize()
        assert s.plan.last_kernel == "k2r_sweep"
        np.testing.assert_array_equal(s.owned((a, b)[ri]).cpu().numpy(), ref)
