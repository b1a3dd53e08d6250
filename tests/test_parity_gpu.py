"""GPU parity: the CUDA path (through the C ABI) against the fp64 oracle,
element by element on seeded inputs, plus bitwise cross-kernel invariants.

Tolerance (north_star; A22): max_p |g_p - o_p| / max(|o_p|, A_p)
<= 1e-5 for one application, <= 1e-4 after 10 iterated steps (Acoustic,
whose field changes sign: |g - o| <= 1e-4 * max|o|).
"""
import itertools

import numpy as np
import pytest
import torch

import stencil_inputs as si
from oracle import stencil_oracle as orc
from stencil_inputs import CLAMP, CONSTANT, MIRROR, REFLECT, WRAP

pytestmark = pytest.mark.gpu

TOL1 = 1e-5
TOL10 = 1e-4
KINDS = [CLAMP, MIRROR, WRAP, CONSTANT, REFLECT]


@pytest.fixture(scope="module")
def lift():
    import __graft_entry__
    __graft_entry__.build()
    import paper_conf_cgo_hagedornssgd18_b200 as m
    torch.cuda.set_device(0)
    return m


def spec(extents, size, weights=None, kind=CLAMP, lo=None, hi=None, step=None, value=0.0,
         op=si.WEIGHTED, params=()):
    nd = len(extents)
    size = tuple(size) if isinstance(size, (tuple, list)) else (size,) * nd
    lo = tuple(s // 2 for s in size) if lo is None else tuple(lo)
    hi = tuple(s - 1 - l for s, l in zip(size, lo)) if hi is None else tuple(hi)
    kind = (kind,) * nd if isinstance(kind, int) else tuple(kind)
    step = (1,) * nd if step is None else tuple(step)
    return si.StencilSpec(tuple(extents), size, step, lo, hi, kind, value, op,
                          None if weights is None else si.f32(weights), tuple(params))


def run_gpu(lift, sp, xs, variant=None):
    plan = lift.Plan.from_spec(sp)
    if variant is not None:
        plan.set_variant(variant)
    dev = [torch.from_numpy(np.ascontiguousarray(x)).cuda() for x in xs]
    y = plan.apply(*dev)
    torch.cuda.synchronize()
    return y.cpu().numpy(), plan


def check(lift, sp, xs, tol=TOL1, variant=None):
    y, plan = run_gpu(lift, sp, xs, variant)
    Y, A = orc.apply(sp, xs)
    assert y.shape == Y.shape
    err = orc.max_rel_err(y, Y, A)
    assert err <= tol, f"max rel err {err:.3e} > {tol} (variant {plan.variant})"
    return y, plan


def rnd(shape, seed, lo=0.5, hi=1.5):
    return si.uniform(shape, seed, lo, hi)


# ------------------------------------------------------------- 1D ---------
@pytest.mark.parametrize("kind", KINDS)
def test_1d(lift, kind):
    x = rnd((1001,), 1)
    check(lift, spec((1001,), 3, [1, 1, 1], kind, value=0.25), [x])
    check(lift, spec((1001,), 5, [0.1, -0.2, 0.5, 0.3, 0.7], kind, lo=(3,), hi=(1,), step=(2,), value=-1.5), [x])
    check(lift, spec((7,), 4, [1, 2, 3, 4], kind, lo=(9,), hi=(6,), value=2.0), [rnd((7,), 2)])  # pad > n


# ------------------------------------------------------------- 2D ---------
@pytest.mark.parametrize("kind", KINDS)
def test_2d_weighted(lift, kind):
    x = rnd((67, 300), 3)
    check(lift, spec(x.shape, 3, si.weights_j2d5(), kind, value=0.75), [x])
    x = rnd((130, 516), 4)
    check(lift, spec(x.shape, 5, si.weights_gauss5(), kind, value=0.75), [x])
    check(lift, spec(x.shape, 3, si.weights_j2d9(), kind, value=0.75), [x])
    w = np.random.default_rng(5).standard_normal((7, 9)).astype(np.float32)
    check(lift, spec(x.shape, (7, 9), w, kind, value=0.75), [x])


def test_2d_valid_asymmetric_strided(lift):
    x = rnd((61, 203), 6)
    w = np.random.default_rng(7).standard_normal((3, 4)).astype(np.float32)
    check(lift, spec(x.shape, (3, 4), w, CLAMP, lo=(0, 0), hi=(0, 0)), [x])          # valid mode
    check(lift, spec(x.shape, (3, 4), w, MIRROR, lo=(2, 0), hi=(1, 3)), [x])         # asymmetric
    check(lift, spec(x.shape, (3, 4), w, (WRAP, CONSTANT), lo=(1, 2), hi=(1, 1), step=(2, 3), value=0.1), [x])


def test_2d_mixed_kinds(lift):
    x = rnd((70, 132), 8)
    for k0, k1 in itertools.product(KINDS, KINDS):
        check(lift, spec(x.shape, 5, si.weights_gauss5(), (k0, k1), value=-0.5), [x])


def test_srad(lift):
    I = np.exp(rnd((130, 260), 9, 0.0, 1.0)).astype(np.float32)
    sp1 = spec(I.shape, 3, op=si.SRAD1, params=si.params_srad1(si.srad_q0sqr(I)))
    c, _ = check(lift, sp1, [I])
    assert c.min() >= 0 and c.max() <= 1
    sp2 = spec(I.shape, 3, op=si.SRAD2, params=si.params_srad2())
    check(lift, sp2, [c.astype(np.float32), I])
    check(lift, sp2, [rnd(I.shape, 10, 0.0, 1.0), I])


# ------------------------------------------------------------- 3D ---------
@pytest.mark.parametrize("kind", KINDS)
def test_3d_weighted(lift, kind):
    x = rnd((37, 70, 260), 11)
    check(lift, spec(x.shape, 3, si.weights_j3d7(), kind, value=0.3), [x])
    x = rnd((21, 40, 132), 12)
    check(lift, spec(x.shape, 5, si.weights_j3d13(), kind, value=0.3), [x])
    w = np.random.default_rng(13).standard_normal((3, 3, 3)).astype(np.float32)
    check(lift, spec(x.shape, 3, w, kind, value=0.3), [x])


def test_3d_mixed_kinds(lift):
    x = rnd((18, 22, 68), 14)
    for ks in [(CLAMP, WRAP, MIRROR), (CONSTANT, CLAMP, WRAP), (WRAP, CONSTANT, REFLECT), (MIRROR, MIRROR, CONSTANT)]:
        check(lift, spec(x.shape, 3, si.weights_j3d7(), ks, value=0.9), [x])
        check(lift, spec(x.shape, 5, si.weights_j3d13(), ks, value=0.9), [x])


def test_hotspot3d(lift):
    T = rnd((8, 64, 132), 15, 300.0, 350.0)
    P = rnd(T.shape, 16, 0.0, 1e-2)
    check(lift, spec(T.shape, 3, op=si.HOTSPOT3D, params=si.params_hotspot3d()), [T, P])


@pytest.mark.parametrize("pts,sz", [(7, 3), (13, 5)])
def test_acoustic(lift, pts, sz):
    u0 = rnd((20, 36, 132), 17, -1.0, 1.0)
    u1 = rnd(u0.shape, 18, -1.0, 1.0)
    check(lift, spec(u0.shape, sz, op=si.ACOUSTIC, params=si.params_acoustic(pts), kind=CONSTANT), [u0, u1])


# ------------------------------------------------------ edge cases --------
def test_degenerate_extents(lift):
    for shape in [(1, 1, 4), (2, 3, 4), (1, 5, 8), (3, 1, 1)]:
        x = rnd(shape, 19)
        for kind in KINDS:
            check(lift, spec(shape, 3, si.weights_j3d7(), kind, value=0.5), [x])
    check(lift, spec((1, 4), 3, si.weights_j2d5(), MIRROR), [rnd((1, 4), 20)])


def test_unaligned_and_odd_width_fall_back(lift):
    x = rnd((20, 30, 66), 21)          # nx % 4 != 0
    check(lift, spec(x.shape, 3, si.weights_j3d7(), CLAMP), [x])
    big = torch.from_numpy(rnd((20 * 30 * 68 + 1,), 22)).cuda()
    xin = big[1:].view(20, 30, 68)     # 4-byte aligned, not 16-byte aligned
    sp = spec((20, 30, 68), 3, si.weights_j3d7(), CLAMP)
    plan = lift.Plan.from_spec(sp)
    y = plan.apply(xin).cpu().numpy()
    Y, A = orc.apply(sp, [xin.cpu().numpy()])
    assert orc.max_rel_err(y, Y, A) <= TOL1


def test_alias_rejected(lift):
    x = torch.from_numpy(rnd((8, 8, 8), 23)).cuda()
    plan = lift.Plan.from_spec(spec((8, 8, 8), 3, si.weights_j3d7()))
    with pytest.raises(lift.StencilError):
        plan.apply(x, out=x)


# ------------------------------------------ bitwise cross-kernel pins ------
def _variants(plan_nd):
    return ["generic", "tile2d"] if plan_nd == 2 else ["generic", "sweep3d"]


@pytest.mark.parametrize("case", ["j2d5", "gauss", "j3d7", "j3d13", "hotspot", "acoustic13", "srad1", "srad2",
                                  "box27_wrap", "box27_const", "box27_mirror", "box19_wrap", "box19_const",
                                  "box19_clamp"])
def test_kernel_families_bitwise_equal(lift, case):
    """Tiling independence: every kernel family gives the same bits."""
    rng = np.random.default_rng(24)
    if case == "j2d5":
        sp, xs = spec((130, 388), 3, si.weights_j2d5(), MIRROR), [rnd((130, 388), 25)]
    elif case == "gauss":
        sp, xs = spec((130, 388), 5, si.weights_gauss5(), WRAP), [rnd((130, 388), 26)]
    elif case == "j3d7":
        sp, xs = spec((19, 37, 264), 3, si.weights_j3d7(), CLAMP), [rnd((19, 37, 264), 27)]
    elif case == "j3d13":
        sp, xs = spec((19, 37, 136), 5, si.weights_j3d13(), REFLECT), [rnd((19, 37, 136), 28)]
    elif case == "hotspot":
        sp = spec((8, 40, 136), 3, op=si.HOTSPOT3D, params=si.params_hotspot3d())
        xs = [rnd((8, 40, 136), 29, 300, 350), rnd((8, 40, 136), 30, 0, 1e-2)]
    elif case == "acoustic13":
        sp = spec((19, 37, 136), 5, op=si.ACOUSTIC, params=si.params_acoustic(13), kind=CONSTANT)
        xs = [rnd((19, 37, 136), 31, -1, 1), rnd((19, 37, 136), 32, -1, 1)]
    elif case.startswith("box"):
        k = {"wrap": WRAP, "const": CONSTANT, "mirror": MIRROR, "clamp": CLAMP}[case.split("_")[1]]
        w = np.random.default_rng(54).standard_normal((3, 3, 3)).astype(np.float32)
        if case.startswith("box19"):        # zero corners: the 19-point kernel (corner taps skipped)
            w[::2, ::2, ::2] = 0.0
        sp, xs = spec((19, 37, 264), 3, w, (k, k, k), value=0.7), [rnd((19, 37, 264), 55)]
    elif case == "srad1":
        I = np.exp(rnd((130, 264), 33, 0, 1)).astype(np.float32)
        sp, xs = spec(I.shape, 3, op=si.SRAD1, params=si.params_srad1(si.srad_q0sqr(I))), [I]
    else:
        I = np.exp(rnd((130, 264), 34, 0, 1)).astype(np.float32)
        sp, xs = spec(I.shape, 3, op=si.SRAD2, params=si.params_srad2()), [rnd(I.shape, 35, 0, 1), I]
    outs = []
    for v in _variants(sp.ndim):
        y, plan = run_gpu(lift, sp, xs, v)
        assert plan.variant == lift.plan.VARIANTS[v]
        outs.append(y)
    assert len(outs) == 2
    np.testing.assert_array_equal(outs[1], outs[0])
    Y, A = orc.apply(sp, xs)
    assert orc.max_rel_err(outs[1], Y, A) <= TOL1


def test_variant_selection(lift):
    """AUTO must pick the TMA kernels for the configs' shapes (no silent K0)."""
    cases = [(spec((64, 64, 128), 3, si.weights_j3d7()), "sweep3d"),
             (spec((64, 64, 128), 5, si.weights_j3d13(), MIRROR), "sweep3d"),
             (spec((8, 64, 128), 3, op=si.HOTSPOT3D, params=si.params_hotspot3d()), "sweep3d"),
             (spec((16, 64, 128), 5, op=si.ACOUSTIC, params=si.params_acoustic(13), kind=CONSTANT), "sweep3d"),
             (spec((64, 128), 3, si.weights_j2d5()), "tile2d"),
             (spec((64, 128), 5, si.weights_gauss5(), MIRROR), "tile2d"),
             (spec((64, 128), 3, op=si.SRAD1, params=(0.1,)), "tile2d"),
             (spec((64, 128), 3, op=si.SRAD2, params=(0.5,)), "tile2d"),
             (spec((64, 64, 130), 3, si.weights_j3d7()), "gather"),
             (spec((64, 64, 128), 3, np.ones((3, 3, 3), np.float32)), "sweep3d"),
             (spec((64, 64, 128), 5, np.ones((5, 5, 5), np.float32)), "gather"),
             (spec((64, 128), 3, si.weights_j2d5(), step=(2, 2)), "gather"),
             (spec((1000,), 3, [1, 2, 3]), "gather")]
    for sp, v in cases:
        plan = lift.Plan.from_spec(sp)
        assert plan.variant == lift.plan.VARIANTS[v], (sp, v)


def _gather_cases():
    r = np.random.default_rng(81)
    w = lambda *shape: r.standard_normal(shape).astype(np.float32)
    return {
        "1d_s2": (spec((1001,), 5, w(5), MIRROR, lo=(3,), hi=(1,), step=(2,)), [rnd((1001,), 82)]),
        "1d_wide_pad": (spec((7,), 4, w(4), WRAP, lo=(9,), hi=(6,)), [rnd((7,), 83)]),
        "2d_3x3_s2_clamp": (spec((257, 390), 3, w(3, 3), CLAMP, step=(2, 2)), [rnd((257, 390), 84)]),
        "2d_2x2_s2_const": (spec((130, 260), 2, w(2, 2), CONSTANT, lo=(0, 0), hi=(1, 1), step=(2, 2), value=0.4),
                            [rnd((130, 260), 85)]),
        "2d_5x5_s3_reflect": (spec((200, 300), 5, w(5, 5), REFLECT, step=(3, 3)), [rnd((200, 300), 86)]),
        "2d_gauss_sep_s2": (spec((300, 520), 5, si.weights_gauss5(), MIRROR, step=(2, 2)), [rnd((300, 520), 87)]),
        "2d_mixed_s21": (spec((99, 333), 3, w(3, 3), (WRAP, CLAMP), step=(2, 1)), [rnd((99, 333), 88)]),
        "3d_3x3x3_s2": (spec((33, 40, 70), 3, w(3, 3, 3), CLAMP, step=(2, 2, 2)), [rnd((33, 40, 70), 89)]),
        "3d_2x2x2_s2_wrap": (spec((32, 34, 64), 2, w(2, 2, 2), WRAP, lo=(0, 0, 0), hi=(1, 1, 1), step=(2, 2, 2)),
                             [rnd((32, 34, 64), 90)]),
        "3d_box5": (spec((20, 30, 68), 5, w(5, 5, 5), MIRROR), [rnd((20, 30, 68), 91)]),
        "3d_odd_width": (spec((20, 30, 66), 3, si.weights_j3d7(), CONSTANT, value=-0.5), [rnd((20, 30, 66), 92)]),
        "3d_asym": (spec((21, 22, 64), (3, 2, 4), w(3, 2, 4), REFLECT, lo=(2, 0, 1), hi=(0, 1, 2)),
                    [rnd((21, 22, 64), 93)]),
        # DAMPEN pads (reading A29): decay^distance, alone and mixed with CONSTANT / reindexing
        "2d_dampen": (dampen(spec((130, 264), 5, si.weights_gauss5(), si.DAMPEN), 0.5), [rnd((130, 264), 98)]),
        "2d_dampen_const": (dampen(spec((99, 140), 3, w(3, 3), (CONSTANT, si.DAMPEN), value=0.3, step=(2, 1)),
                                   0.75), [rnd((99, 140), 99)]),
        "3d_dampen_mixed": (dampen(spec((20, 26, 68), 3, w(3, 3, 3), (si.DAMPEN, CONSTANT, si.DAMPEN),
                                        lo=(2, 1, 3), hi=(1, 2, 2), value=-0.2), 0.6), [rnd((20, 26, 68), 100)]),
        "3d_dampen_star": (dampen(spec((24, 40, 136), 3, si.weights_j3d7(), (si.DAMPEN, WRAP, si.DAMPEN)), 0.9),
                           [rnd((24, 40, 136), 101)]),
        "1d_dampen": (dampen(spec((500,), 5, w(5), si.DAMPEN, lo=(4,), hi=(3,)), 0.3), [rnd((500,), 102)]),
    }


def dampen(sp, decay):
    sp.pad_decay = decay
    return sp


@pytest.mark.parametrize("case", list(_gather_cases()))
def test_gather_kernel(lift, case):
    """K5 (shared-memory input boxes) for WEIGHTED plans the TMA families do
    not take: parity with the oracle and bitwise equality with K0."""
    sp, xs = _gather_cases()[case]
    y, plan = check(lift, sp, xs)
    assert plan.variant == lift.plan.VARIANTS["gather"]
    y0, p0 = run_gpu(lift, sp, xs, "generic")
    assert p0.variant == 0
    np.testing.assert_array_equal(y, y0)


def test_gather_apply_region_pieces(lift):
    x = rnd((41, 36, 70), 94)
    sp = spec(x.shape, 3, np.random.default_rng(95).standard_normal((3, 3, 3)).astype(np.float32), MIRROR,
              step=(2, 1, 2))
    full, plan = run_gpu(lift, sp, [x])
    assert plan.variant == lift.plan.VARIANTS["gather"]
    xd = torch.from_numpy(x).cuda()
    o = sp.out_extents()
    out = torch.full(o, float("nan"), device="cuda")
    for a, b in [(0, 1), (1, 6), (6, 20), (20, o[0])]:
        plan.apply_region(xd, out=out, begin=a, end=b)
    torch.cuda.synchronize()
    np.testing.assert_array_equal(out.cpu().numpy(), full)


def test_apply_region_pieces_bitwise(lift):
    x = rnd((33, 40, 136), 36)
    sp = spec(x.shape, 3, si.weights_j3d7(), CLAMP)
    full, plan = run_gpu(lift, sp, [x])
    xd = torch.from_numpy(x).cuda()
    out = torch.full(x.shape, float("nan"), device="cuda")
    for a, b in [(0, 1), (1, 7), (7, 32), (32, 33)]:
        plan.apply_region(xd, out=out, begin=a, end=b)
    torch.cuda.synchronize()
    np.testing.assert_array_equal(out.cpu().numpy(), full)


def test_constant_field_bitwise(lift):
    for sp_ in [spec((9, 40, 132), 3, [[[0, 0, 0], [0, .125, 0], [0, 0, 0]],
                                       [[0, .125, 0], [.125, .25, .125], [0, .125, 0]],
                                       [[0, 0, 0], [0, .125, 0], [0, 0, 0]]], WRAP),
                spec((70, 132), 5, si.weights_gauss5(), MIRROR)]:
        x = np.full(sp_.extents, 0.8125, np.float32)
        y, _ = run_gpu(lift, sp_, [x])
        assert np.all(y == np.float32(0.8125))


def test_wrap_translation_bitwise(lift):
    x = rnd((16, 36, 132), 37)
    sp = spec(x.shape, 3, si.weights_j3d7(), WRAP)
    y, _ = run_gpu(lift, sp, [x])
    ys, _ = run_gpu(lift, sp, [np.ascontiguousarray(np.roll(x, (3, -5, 8), axis=(0, 1, 2)))])
    np.testing.assert_array_equal(ys, np.roll(y, (3, -5, 8), axis=(0, 1, 2)))


# ------------------------------------------------------------ iterate -----
def test_iterate_weighted_10_steps(lift):
    x = rnd((24, 40, 136), 38)
    sp = spec(x.shape, 3, si.weights_j3d7(), CLAMP)
    plan = lift.Plan.from_spec(sp)
    a = torch.from_numpy(x).cuda()
    b = torch.empty_like(a)
    ri = plan.iterate([a, b], 10)
    g = (a, b)[ri].cpu().numpy()
    ref = orc.iterate(sp, [x], [], 10)[0]
    assert np.max(np.abs(g - ref) / np.abs(ref)) <= TOL10
    # iterate == 10 x apply with the same rotation, bitwise
    c = torch.from_numpy(x).cuda()
    d = torch.empty_like(c)
    for _ in range(10):
        plan.apply(c, out=d)
        c, d = d, c
    torch.cuda.synchronize()
    np.testing.assert_array_equal(c.cpu().numpy(), g)


def test_iterate_hotspot_10_steps(lift):
    T = rnd((8, 40, 136), 39, 300, 350)
    P = rnd(T.shape, 40, 0, 1e-2)
    sp = spec(T.shape, 3, op=si.HOTSPOT3D, params=si.params_hotspot3d())
    plan = lift.Plan.from_spec(sp)
    a, b, p = (torch.from_numpy(v).cuda() for v in (T, np.empty_like(T), P))
    ri = plan.iterate([a, b], 10, aux=[p])
    g = (a, b)[ri].cpu().numpy()
    ref = orc.iterate(sp, [T], [P], 10)[0]
    assert np.max(np.abs(g - ref) / np.abs(ref)) <= TOL10


@pytest.mark.parametrize("pts,sz", [(7, 3), (13, 5)])
def test_iterate_acoustic_10_steps(lift, pts, sz):
    u = rnd((20, 36, 132), 41, -1, 1)
    sp = spec(u.shape, sz, op=si.ACOUSTIC, params=si.params_acoustic(pts), kind=CONSTANT)
    plan = lift.Plan.from_spec(sp)
    a = torch.from_numpy(u).cuda()
    b = torch.from_numpy(u.copy()).cuda()
    ri = plan.iterate([a, b], 10)
    g = (a, b)[ri].cpu().numpy()
    ref = orc.iterate(sp, [u, u], [], 10)[1]
    assert np.max(np.abs(g - ref)) <= TOL10 * np.max(np.abs(ref))


def test_run_host_matches_device(lift):
    x = rnd((24, 40, 136), 42)
    sp = spec(x.shape, 3, si.weights_j3d7(), MIRROR)
    plan = lift.Plan.from_spec(sp)
    a = torch.from_numpy(x).cuda()
    b = torch.empty_like(a)
    ri = plan.iterate([a, b], 3)
    dev = (a, b)[ri].cpu().numpy()
    host = plan.run_host([x], n_steps=3)
    np.testing.assert_array_equal(host, dev)


# ------------------------------------------------ Table 1 extras (NEXT-1) --
@pytest.mark.parametrize("kind", [CLAMP, MIRROR, WRAP])
def test_hotspot2d_and_gradient(lift, kind):
    T = rnd((100, 260), 50, 300.0, 350.0)
    P = rnd(T.shape, 51, 0.0, 1e-2)
    sp = spec(T.shape, 3, op=si.HOTSPOT2D, params=si.params_hotspot2d(512, 512), kind=kind)
    y, plan = check(lift, sp, [T, P])
    assert plan.variant == 1
    y0, _ = run_gpu(lift, sp, [T, P], "generic")
    np.testing.assert_array_equal(y, y0)
    I = rnd((100, 260), 52, 0.0, 1.0)
    sp = spec(I.shape, 3, op=si.GRADIENT, params=si.params_gradient(), kind=kind)
    y, plan = check(lift, sp, [I])
    assert plan.variant == 1
    y0, _ = run_gpu(lift, sp, [I], "generic")
    np.testing.assert_array_equal(y, y0)


def test_poisson19_and_heat7(lift):
    x = rnd((20, 40, 132), 53)
    check(lift, spec(x.shape, 3, si.weights_poisson19(), MIRROR), [x])
    _, plan = check(lift, spec(x.shape, 3, si.weights_heat7(), CLAMP), [x])
    assert plan.variant == 2


# ------------------------------------------- temporal blocking (NEXT-3) ----
@pytest.mark.parametrize("kind", [CLAMP, MIRROR, REFLECT])
@pytest.mark.parametrize("shape", [(37, 70, 260), (3, 15, 124), (1, 14, 120), (2, 29, 244), (40, 8, 516)])
def test_time_block2_bitwise_equal_single_steps(lift, kind, shape):
    """Two steps per pass (K2T) give exactly the bits of single steps."""
    x = rnd(shape, 60)
    sp = spec(shape, 3, si.weights_j3d7(), kind)
    res = {}
    for tb in (1, 2):
        plan = lift.Plan.from_spec(sp)
        plan.set_time_block(tb)
        assert plan.time_block == tb
        a = torch.from_numpy(x).cuda()
        b = torch.empty_like(a)
        ri = plan.iterate([a, b], 7)
        res[tb] = (a, b)[ri].cpu().numpy()
    np.testing.assert_array_equal(res[2], res[1])
    ref = orc.iterate(sp, [x], [], 7)[0]
    assert np.max(np.abs(res[2] - ref) / np.abs(ref)) <= TOL10


def test_time_block_eligibility(lift):
    # (plan, default AUTO, after set_time_block(2)): AUTO takes two steps per
    # pass exactly where K2R applies (z CLAMP / MIRROR); 2 also takes K2T (z REFLECT)
    # (AUTO also needs a grid that fills the GPU: >= 8 tiles of 128 x 48, >= 2048 (plane, tile) pairs)
    for sp_, auto, exp in [(spec((128, 256, 512), 3, si.weights_j3d7()), 2, 2),
                           (spec((64, 64, 128), 3, si.weights_j3d7()), 1, 2),
                           (spec((64, 64, 128), 3, si.weights_j3d7(), (REFLECT, CLAMP, CLAMP)), 1, 2),
                           (spec((64, 64, 128), 3, si.weights_j3d7(), WRAP), 1, 1),
                           (spec((64, 64, 128), 5, si.weights_j3d13()), 1, 1)]:
        plan = lift.Plan.from_spec(sp_)
        assert plan.time_block == auto
        plan.set_time_block(2)
        assert plan.time_block == exp
        plan.set_time_block(1)
        assert plan.time_block == 1


# ---------------------------------------- full SRAD iteration (NEXT-2) -----
@pytest.mark.parametrize("kind", [CLAMP, MIRROR, REFLECT, WRAP, (WRAP, CLAMP), (MIRROR, WRAP)])
def test_srad_iteration(lift, kind):
    """q0 reduction + SRAD1/SRAD2 fused in one pass (K1S) vs the oracle's
    SRAD1-then-SRAD2 with q0 of the current image; K1S == K0 bitwise."""
    I = np.exp(rnd((150, 388), 61, 0.0, 1.0)).astype(np.float32)
    sp = spec(I.shape, 3, op=si.SRAD, params=si.params_srad2(), kind=kind)
    y, plan = check(lift, sp, [I])
    assert plan.variant == 1
    y0, _ = run_gpu(lift, sp, [I], "generic")
    np.testing.assert_array_equal(y, y0)
    # 10 iterations
    a = torch.from_numpy(I).cuda()
    b = torch.empty_like(a)
    ri = plan.iterate([a, b], 10)
    g = (a, b)[ri].cpu().numpy()
    ref = orc.iterate(sp, [I], [], 10)[0]
    assert np.max(np.abs(g - ref) / np.abs(ref)) <= TOL10


@pytest.mark.parametrize("shape", [(2500, 2052), (97, 260)])
def test_srad_iterate_chain(lift, shape):
    """stencil_iterate hands each fused pass's q0 statistics (per-CTA fp64
    partials of the image it wrote) to the next pass instead of re-reducing
    the image: the chain agrees with step-by-step applies (each reducing its
    own input) to fp64-sum rounding, and with the oracle after 6 iterations.
    (2500, 2052): more tiles than resident CTAs, ragged in y."""
    I = np.exp(rnd(shape, 63, 0.0, 1.0)).astype(np.float32)
    sp = spec(I.shape, 3, op=si.SRAD, params=si.params_srad2(), kind=CLAMP)
    plan = lift.Plan.from_spec(sp)
    a = torch.from_numpy(I).cuda()
    b = torch.empty_like(a)
    ri = plan.iterate([a, b], 6)
    assert plan.variant == 1
    g = (a, b)[ri].cpu().numpy()
    x = torch.from_numpy(I).cuda()
    for _ in range(6):
        x = plan.apply(x)
    h = x.cpu().numpy()
    assert np.max(np.abs(g - h) / np.abs(h)) <= 1e-6
    ref = orc.iterate(sp, [I], [], 6)[0]
    assert np.max(np.abs(g - ref) / np.abs(ref)) <= TOL10


@pytest.mark.parametrize("case,steps", [("clamp", 10), ("wrap", 7), ("const", 10), ("mirror", 3), ("hotspot", 10),
                                        ("hotspot_reflect", 5), ("ragged", 6)])
def test_persistent_iterate_bitwise(lift, case, steps, monkeypatch):
    """K4 — all time steps of a small (L2-resident) 3D grid in one cooperative
    launch with grid barriers — gives the bits of step-by-step K2 launches,
    and matches the oracle after the steps (odd counts: result in state[1])."""
    monkeypatch.setenv("LIFT_K4", "1")          # K4 is opt-in (measured slower than K2 steps)
    shape = (11, 13, 52) if case == "ragged" else (12, 36, 136)
    if case == "ragged":
        case = "clamp"
    if case.startswith("hotspot"):
        kind = REFLECT if case.endswith("reflect") else CLAMP
        sp = spec(shape, 3, op=si.HOTSPOT3D, params=si.params_hotspot3d(), kind=kind)
        xs, aux = [rnd(shape, 71, 300, 350)], [rnd(shape, 72, 0, 1e-2)]
    else:
        k = {"clamp": CLAMP, "wrap": WRAP, "const": CONSTANT, "mirror": MIRROR}[case]
        sp = spec(shape, 3, si.weights_j3d7(), k, value=0.3)
        xs, aux = [rnd(shape, 73)], []
    outs = []
    for variant, fam in [(None, 3), ("sweep3d", 2)]:
        plan = lift.Plan.from_spec(sp)
        if variant:
            plan.set_variant(variant)
            plan.set_time_block(1)          # K4 vs one K2 launch per step
        a = torch.from_numpy(xs[0].copy()).cuda()
        b = torch.empty_like(a)
        dev_aux = [torch.from_numpy(x).cuda() for x in aux]
        ri = plan.iterate([a, b], steps, aux=dev_aux)
        torch.cuda.synchronize()
        assert plan.last_variant == fam
        assert ri == steps % 2
        outs.append((a, b)[ri].cpu().numpy())
    np.testing.assert_array_equal(outs[0], outs[1])
    ref = orc.iterate(sp, xs, aux, steps)[0]
    assert np.max(np.abs(outs[0] - ref) / np.maximum(np.abs(ref), 1e-3)) <= TOL10


def test_cuda_graph_capture_replay(lift):
    """apply / iterate allocate nothing and are stream-ordered: captured into a
    CUDA graph, replays give the same bits as eager calls (stencil.h)."""
    x = rnd((24, 40, 136), 62)
    sp = spec(x.shape, 3, si.weights_j3d7(), CLAMP)
    plan = lift.Plan.from_spec(sp)
    a = torch.from_numpy(x).cuda()
    b = torch.empty_like(a)
    c = torch.empty_like(a)
    s = torch.cuda.Stream()
    s.wait_stream(torch.cuda.current_stream())
    with torch.cuda.stream(s):
        plan.apply(a, out=b)                       # warm-up (TMA descriptors, function attributes)
    torch.cuda.current_stream().wait_stream(s)
    g = torch.cuda.CUDAGraph()
    with torch.cuda.graph(g):
        plan.apply(a, out=b)
        plan.iterate([b, c], 4)
    for _ in range(3):
        g.replay()
    torch.cuda.synchronize()
    e1 = plan.apply(a)
    e2 = torch.empty_like(a)
    ri = plan.iterate([e1, e2], 4)
    torch.cuda.synchronize()
    np.testing.assert_array_equal((b, c)[ri].cpu().numpy(), (e1, e2)[ri].cpu().numpy())


# --------------------------- K1 with cp.async fill (nx % 4 != 0, unaligned) --
@pytest.mark.parametrize("shape", [(67, 301), (45, 258), (50, 4098 // 8 + 1)])
def test_tile2d_unaligned_widths(lift, shape):
    x = rnd(shape, 63)
    I = np.exp(rnd(shape, 64, 0, 1)).astype(np.float32)
    cases = [(spec(shape, 3, si.weights_j2d5(), MIRROR), [x]),
             (spec(shape, 5, si.weights_gauss5(), CLAMP), [x]),
             (spec(shape, 3, si.weights_j2d9(), WRAP), [x]),
             (spec(shape, 3, op=si.SRAD1, params=si.params_srad1(si.srad_q0sqr(I))), [I]),
             (spec(shape, 3, op=si.HOTSPOT2D, params=si.params_hotspot2d(512, 512)), [x * 300, x * 1e-2]),
             (spec(shape, 3, op=si.GRADIENT, params=si.params_gradient()), [x])]
    for sp_, xs in cases:
        y, plan = check(lift, sp_, xs)
        assert plan.variant == 1, sp_
        y0, _ = run_gpu(lift, sp_, xs, "generic")
        np.testing.assert_array_equal(y, y0)


@pytest.mark.parametrize("off,shape,kind", [(1, (70, 264), MIRROR),      # 4-byte aligned only: 4-B fill
                                             (2, (70, 264), MIRROR),      # 8-byte aligned: pair fill
                                             (2, (37, 4098 // 16 * 2 + 2), CONSTANT)])
def test_tile2d_unaligned_pointer(lift, off, shape, kind):
    n = shape[0] * shape[1]
    big = torch.from_numpy(rnd((n + off,), 65)).cuda()
    xin = big[off:].view(*shape)
    sp = spec(shape, 5, si.weights_gauss5(), kind, value=-0.25)
    plan = lift.Plan.from_spec(sp)
    out_big = torch.empty(n + 3, device="cuda")
    out = out_big[3:].view(*shape)
    plan.apply(xin, out=out)
    torch.cuda.synchronize()
    assert plan.variant == 1
    Y, A = orc.apply(sp, [xin.cpu().numpy()])
    assert orc.max_rel_err(out.cpu().numpy(), Y, A) <= TOL1


# ------------------------------------------------- K3 per-warp sweeps ------
@pytest.mark.parametrize("case", ["j2d5", "gauss", "box", "srad1", "srad2", "hot2d", "grad"])
@pytest.mark.parametrize("kind", [CLAMP, MIRROR, REFLECT, CONSTANT, WRAP])
def test_wsweep2d_bitwise_vs_k1_k0(lift, case, kind, monkeypatch):
    """K3 (per-warp y-sweeps) against K1 (tiles) and K0 (generic), bitwise, for
    several rows-per-item values (one group, several sweep blocks, a ragged
    last chunk) and ragged strips; WRAP in y runs K3 with remapped rows."""
    shape = (203, 392)          # 4 strips, the last 8 columns wide
    kinds = (kind, CLAMP if kind == WRAP else kind)     # WRAP in x runs on K1
    if case == "j2d5":
        sp, xs = spec(shape, 3, si.weights_j2d5(), kinds, value=0.75), [rnd(shape, 60)]
    elif case == "gauss":
        sp, xs = spec(shape, 5, si.weights_gauss5(), kinds, value=0.75), [rnd(shape, 61)]
    elif case == "box":
        w = np.random.default_rng(62).standard_normal((5, 3)).astype(np.float32)
        sp, xs = spec(shape, (5, 3), w, kinds, value=-0.5), [rnd(shape, 63)]
    elif case == "srad1":
        I = np.exp(rnd(shape, 64, 0, 1)).astype(np.float32)
        sp, xs = spec(shape, 3, op=si.SRAD1, params=si.params_srad1(si.srad_q0sqr(I)), kind=kinds, value=1.5), [I]
    elif case == "srad2":
        I = np.exp(rnd(shape, 65, 0, 1)).astype(np.float32)
        sp, xs = spec(shape, 3, op=si.SRAD2, params=si.params_srad2(), kind=kinds, value=0.5), [rnd(shape, 66, 0, 1), I]
    elif case == "hot2d":
        sp = spec(shape, 3, op=si.HOTSPOT2D, params=si.params_hotspot2d(*shape), kind=kinds, value=320.0)
        xs = [rnd(shape, 67, 300, 350), rnd(shape, 68, 0, 1e-2)]
    else:
        sp, xs = spec(shape, 3, op=si.GRADIENT, params=si.params_gradient(), kind=kinds, value=0.5), [rnd(shape, 69)]
    y0, plan = run_gpu(lift, sp, xs, "generic")
    monkeypatch.setenv("LIFT_K3", "0")
    y1, _ = run_gpu(lift, sp, xs, "tile2d")
    np.testing.assert_array_equal(y1, y0)
    monkeypatch.setenv("LIFT_K3", "1")
    for hc in ("1", "6", "14", "61", "203", "512"):
        monkeypatch.setenv("LIFT_K3_HC", hc)
        y, plan = run_gpu(lift, sp, xs, "tile2d")
        np.testing.assert_array_equal(y, y0, err_msg=f"hc={hc}")
    Y, A = orc.apply(sp, xs)
    assert orc.max_rel_err(y0, Y, A) <= TOL1


# ------------------------------------- K2C whole-column tiles (nz <= 16) ----
K2C_SHAPES = [(1, 20, 132), (2, 9, 128), (3, 33, 260), (8, 64, 132), (16, 17, 516)]


@pytest.mark.parametrize("shape", K2C_SHAPES)
@pytest.mark.parametrize("kind", KINDS)
@pytest.mark.parametrize("op", ["j3d7", "hotspot"])
def test_column3d_few_planes(lift, monkeypatch, shape, kind, op):
    """Few-plane 3D grids run on K2C (one TMA box per CTA over all nz planes):
    parity with the oracle, bitwise equal to K0 and to the K2 ring sweep
    (LIFT_K2C=0), every pad kind, ragged x/y tiles, nz = 1 .. 16."""
    if op == "j3d7":
        xs = [rnd(shape, 141)]
        sp = spec(shape, 3, si.weights_j3d7(), kind, value=0.75)
    else:
        xs = [rnd(shape, 142, 300.0, 350.0), rnd(shape, 143, 0.0, 1e-2)]
        sp = spec(shape, 3, op=si.HOTSPOT3D, params=si.params_hotspot3d(), kind=kind, value=0.75)
    y, plan = check(lift, sp, xs)
    assert plan.last_variant == 2
    y0, _ = run_gpu(lift, sp, xs, "generic")
    np.testing.assert_array_equal(y, y0)
    monkeypatch.setenv("LIFT_K2C", "0")
    y2, _ = run_gpu(lift, sp, xs)
    np.testing.assert_array_equal(y, y2)


def test_column3d_iterate_hotspot(lift, monkeypatch):
    """Hotspot3D iterate (the x100 workload's structure) on K2C == K2 ring bitwise."""
    T = rnd((8, 96, 264), 144, 300.0, 350.0)
    P = rnd(T.shape, 145, 0.0, 1e-2)
    sp = spec(T.shape, 3, op=si.HOTSPOT3D, params=si.params_hotspot3d())
    plan = lift.Plan.from_spec(sp)
    outs = []
    for env in ("1", "0"):
        monkeypatch.setenv("LIFT_K2C", env)
        a, b = torch.from_numpy(T).cuda(), torch.empty(T.shape, device="cuda")
        ri = plan.iterate([a, b], 9, [torch.from_numpy(P).cuda()])
        outs.append((a, b)[ri].cpu().numpy())
    np.testing.assert_array_equal(outs[0], outs[1])
    ref = orc.iterate(sp, [T], [P], 9)[0]
    assert np.max(np.abs(outs[0] - ref) / np.abs(ref)) <= TOL10


# ------------------------------- K6 shared-memory-resident iterate ----------
K6_SHAPES = [(8, 512, 512), (8, 96, 264), (1, 40, 128), (3, 130, 388), (16, 64, 132)]


@pytest.mark.parametrize("shape", K6_SHAPES)
@pytest.mark.parametrize("kind", KINDS)
@pytest.mark.parametrize("op", ["j3d7", "hotspot"])
def test_resident3d_iterate(lift, monkeypatch, shape, kind, op):
    """K6 (opt-in; the whole grid in shared memory, one cooperative launch,
    step flags between neighbour tiles): bitwise equal to stepping K2C/K2
    launches (LIFT_K6=0)
    for 2, 5 and 9 steps, and within the 10-step tolerance of the oracle."""
    if op == "j3d7":
        xs, aux = [rnd(shape, 151)], []
        sp = spec(shape, 3, si.weights_j3d7(), kind, value=0.75)
    else:
        xs, aux = [rnd(shape, 152, 300.0, 350.0)], [rnd(shape, 153, 0.0, 1e-2)]
        sp = spec(shape, 3, op=si.HOTSPOT3D, params=si.params_hotspot3d(), kind=kind, value=0.75)
    plan = lift.Plan.from_spec(sp)
    for n in (2, 5, 9):
        res = {}
        for env in ("1", "0"):
            monkeypatch.setenv("LIFT_K6", env)          # K6 is opt-in
            a, b = torch.from_numpy(xs[0]).cuda(), torch.empty(shape, device="cuda")
            ri = plan.iterate([a, b], n, [torch.from_numpy(x).cuda() for x in aux])
            torch.cuda.synchronize()
            if env == "1":
                assert ri == n % 2          # (AUTO two-step passes may leave the result elsewhere)
            res[env] = ((a, b)[ri].cpu().numpy(), plan.last_variant)
        assert res["1"][1] == lift.plan.VARIANTS["resident3d"]
        assert res["0"][1] != lift.plan.VARIANTS["resident3d"]
        np.testing.assert_array_equal(res["1"][0], res["0"][0], err_msg=f"{n} steps")
    if int(np.prod(shape)) <= 1 << 20:
        ref = orc.iterate(sp, xs, aux, 9)[0]
        Y = res["1"][0].astype(np.float64)
        assert np.max(np.abs(Y - ref) / np.maximum(np.abs(ref), 1e-30)) <= TOL10


# --------------------------- K5 TMA box fill (interior tiles) ---------------
K5_TMA_CASES = {
    "2d_3x3_s2": ((260, 520), (3, 3), (2, 2), (1, 1), (1, 1), (MIRROR, CLAMP)),
    "2d_5x5_s2": ((300, 1032), (5, 5), (2, 2), (2, 2), (2, 2), (REFLECT, WRAP)),
    "2d_2x2_s2": ((256, 512), (2, 2), (2, 2), (0, 0), (1, 1), (CLAMP, CLAMP)),
    "2d_4x3_s3x2": ((301, 516), (4, 3), (3, 2), (1, 1), (2, 1), (CONSTANT, MIRROR)),
    "3d_2x2x2_s2": ((40, 72, 264), (2, 2, 2), (2, 2, 2), (0, 0, 0), (1, 1, 1), (CLAMP, WRAP, MIRROR)),
    "3d_3x2x4_s1x2x2": ((20, 40, 520), (3, 2, 4), (1, 2, 2), (1, 0, 1), (1, 1, 2), (REFLECT, CLAMP, CONSTANT)),
}


@pytest.mark.parametrize("case", list(K5_TMA_CASES))
def test_k5_tma_interior_tiles(lift, monkeypatch, case):
    """K5 boxes fully inside the grid arrive as one TMA load, edge boxes
    through the warps' cp.async fill: both are bitwise K0 and the cp.async-only
    build (LIFT_K5_TMA=0), and match the oracle (grids several tiles wide,
    nx % 4 == 0 so TMA applies; mixed pads; strided and asymmetric windows)."""
    ext, size, step, lo, hi, kinds = K5_TMA_CASES[case]
    w = np.random.default_rng(161).standard_normal(size).astype(np.float32)
    sp = spec(ext, size, w, kinds, lo=lo, hi=hi, step=step, value=0.3)
    xs = [rnd(ext, 162)]
    y, plan = check(lift, sp, xs)
    assert plan.last_variant == lift.plan.VARIANTS["gather"]
    y0, _ = run_gpu(lift, sp, xs, "generic")
    np.testing.assert_array_equal(y, y0)
    monkeypatch.setenv("LIFT_K5_TMA", "0")
    y1, _ = run_gpu(lift, sp, xs)
    np.testing.assert_array_equal(y, y1)


def test_last_kernel_names(lift, monkeypatch):
    """stencil_plan_last_kernel names the kernel function within a family."""
    T = rnd((8, 64, 132), 171, 300.0, 350.0)
    P = rnd(T.shape, 172, 0.0, 1e-2)
    sp = spec(T.shape, 3, op=si.HOTSPOT3D, params=si.params_hotspot3d())
    y, plan = run_gpu(lift, sp, [T, P])
    assert plan.last_kernel == "k2c_column"
    monkeypatch.setenv("LIFT_K2C", "0")
    y, plan = run_gpu(lift, sp, [T, P])
    assert plan.last_kernel == "k2_sweep"
    x = rnd((40, 48, 136), 173)
    y, plan = run_gpu(lift, spec(x.shape, 3, si.weights_j3d7()), [x])
    assert plan.last_kernel == "k2_sweep"
    y, plan = run_gpu(lift, spec(x.shape, 3, si.weights_j3d7()), [x], "generic")
    assert plan.last_kernel == "k0_generic"
    x2 = rnd((260, 520), 174)
    y, plan = run_gpu(lift, spec(x2.shape, (3, 3), np.ones((3, 3), np.float32) / 9, step=(2, 2)), [x2])
    assert plan.last_kernel == "k5_gather (TMA)"
    I = np.exp(rnd((150, 388), 175, 0.0, 1.0)).astype(np.float32)
    y, plan = run_gpu(lift, spec(I.shape, 3, op=si.SRAD, params=si.params_srad2()), [I])
    assert plan.last_kernel == "k1_srad_fused"
