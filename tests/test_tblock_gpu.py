"""K2R — two weighted 7-point steps per pass with X_{t+1} in registers
(temporal blocking; tiling preserves semantics, PAPER.md
P:771-791): bitwise equal to single steps and within the iterate tolerance of
the fp64 oracle, over tile / chunk / boundary cases.

Tiles are 128 columns x 8*RPW rows (RPW = 8 by default; LIFT_K2R_SHAPE=4/6
picks the other instantiations), z-chunks are chosen by the launcher
(LIFT_K2R_ZC / LIFT_K2R_ZC2 force them: every chunk boundary recomputes two
X_{t+1} planes).
"""
import os

import numpy as np
import pytest
import torch

import stencil_inputs as si
from oracle import stencil_oracle as orc
from stencil_inputs import CLAMP, MIRROR, REFLECT, WRAP

pytestmark = pytest.mark.gpu

TOL10 = 1e-4


@pytest.fixture(scope="module")
def lift():
    import __graft_entry__
    __graft_entry__.build()
    import paper_conf_cgo_hagedornssgd18_b200 as m
    torch.cuda.set_device(0)
    return m


def rnd(shape, seed):
    return np.random.default_rng(seed).uniform(0.5, 1.5, size=shape).astype(np.float32)


def spec(extents, kind):
    kind = (kind,) * 3 if isinstance(kind, int) else tuple(kind)
    return si.StencilSpec(tuple(extents), (3, 3, 3), (1, 1, 1), (1, 1, 1), (1, 1, 1), kind, 0.0,
                          si.WEIGHTED, si.f32(si.weights_j3d7()), ())


def run(lift, sp, x, steps, tb, env=None):
    old = {}
    for k, v in (env or {}).items():
        old[k] = os.environ.get(k)
        os.environ[k] = v
    try:
        plan = lift.Plan.from_spec(sp)
        plan.set_time_block(tb)
        a = torch.from_numpy(x).cuda()
        b = torch.empty_like(a)
        ri = plan.iterate([a, b], steps)
        torch.cuda.synchronize()
        return (a, b)[ri].cpu().numpy(), plan
    finally:
        for k, v in old.items():
            if v is None:
                os.environ.pop(k, None)
            else:
                os.environ[k] = v


SHAPES = [(37, 70, 260), (3, 15, 124), (1, 14, 120), (2, 129, 244), (40, 8, 516), (5, 1, 128),
          (4, 2, 132), (9, 65, 128), (6, 64, 256), (17, 130, 388), (2, 3, 4)]


@pytest.mark.parametrize("kind", [CLAMP, MIRROR, (CLAMP, REFLECT, REFLECT), (MIRROR, CLAMP, REFLECT),
                                  (CLAMP, MIRROR, CLAMP)])
@pytest.mark.parametrize("shape", SHAPES)
def test_k2r_bitwise_equal_single_steps(lift, kind, shape):
    x = rnd(shape, 70)
    sp = spec(shape, kind)
    y1, _ = run(lift, sp, x, 6, 1)
    y2, plan = run(lift, sp, x, 6, 2)
    assert plan.time_block == 2
    assert plan.last_kernel == "k2r_sweep"
    np.testing.assert_array_equal(y2, y1)


@pytest.mark.parametrize("rpw", ["4", "6", "8"])
@pytest.mark.parametrize("zc", [("1", "0"), ("2", "0"), ("3", "1"), ("5", "2"), ("64", "0")])
def test_k2r_shapes_and_chunks(lift, rpw, zc):
    shape = (23, 70, 260)
    x = rnd(shape, 71)
    for kind in (CLAMP, (MIRROR, REFLECT, MIRROR)):
        sp = spec(shape, kind)
        y1, _ = run(lift, sp, x, 4, 1)
        y2, plan = run(lift, sp, x, 4, 2, {"LIFT_K2R_SHAPE": rpw, "LIFT_K2R_ZC": zc[0], "LIFT_K2R_ZC2": zc[1]})
        assert plan.last_kernel == "k2r_sweep"
        np.testing.assert_array_equal(y2, y1)


def test_k2r_odd_steps_vs_oracle(lift):
    shape = (19, 37, 132)
    x = rnd(shape, 72)
    sp = spec(shape, CLAMP)
    y2, _ = run(lift, sp, x, 7, 2)            # three K2R passes + one single step
    ref = orc.iterate(sp, [x], [], 7)[0]
    assert np.max(np.abs(y2 - ref) / np.abs(ref)) <= TOL10
    y1, _ = run(lift, sp, x, 7, 1)
    np.testing.assert_array_equal(y2, y1)


def test_k2r_not_taken(lift):
    """z REFLECT (the out-of-grid X_{t+1} plane is not the edge plane) keeps
    the shared-memory two-step kernel; WRAP keeps single steps."""
    shape = (12, 20, 128)
    x = rnd(shape, 73)
    sp = spec(shape, (REFLECT, CLAMP, CLAMP))
    y2, plan = run(lift, sp, x, 4, 2)
    assert plan.last_kernel == "k2t_sweep"
    y1, _ = run(lift, sp, x, 4, 1)
    np.testing.assert_array_equal(y2, y1)
    sp = spec(shape, WRAP)
    plan = lift.Plan.from_spec(sp)
    plan.set_time_block(2)
    assert plan.time_block == 1


def test_k2r_j3d7_512_sampled(lift):
    """BASELINE C3 size (512^3, clamp), 10 steps as 5 K2R passes: bitwise equal
    to single steps over the whole grid."""
    xs, sp = si.make_workload_inputs(si.workload("j3d7_512_clamp"))
    y1, _ = run(lift, sp, xs[0], 10, 1)
    y2, plan = run(lift, sp, xs[0], 10, 2)
    assert plan.last_kernel == "k2r_sweep"
    assert np.array_equal(y2, y1)


# ------------------------------------------------------------------ K2RA ----
# Two Acoustic steps per pass (Listing 3; zero padding): iterate
# with four state buffers {prev, cur, spare, spare}; the newest grid is
# state[ri], the one before it state[ri ^ 1].

def ac_spec(extents, pts):
    return si.StencilSpec(tuple(extents), (5, 5, 5) if pts == 13 else (3, 3, 3), (1, 1, 1),
                          (2, 2, 2) if pts == 13 else (1, 1, 1), (2, 2, 2) if pts == 13 else (1, 1, 1),
                          (si.CONSTANT,) * 3, 0.0, si.ACOUSTIC, None, si.params_acoustic(pts))


def ac_run(lift, sp, u0, u1, steps, nbuf, env=None, tb=2):
    old = {}
    for k, v in (env or {}).items():
        old[k] = os.environ.get(k)
        os.environ[k] = v
    try:
        plan = lift.Plan.from_spec(sp)
        plan.set_time_block(tb)
        bufs = [torch.from_numpy(u0.copy()).cuda(), torch.from_numpy(u1.copy()).cuda()]
        bufs += [torch.full_like(bufs[0], float("nan")) for _ in range(nbuf - 2)]
        ri = plan.iterate(bufs, steps)
        torch.cuda.synchronize()
        return bufs[ri].cpu().numpy(), bufs[ri ^ 1].cpu().numpy(), plan
    finally:
        for k, v in old.items():
            if v is None:
                os.environ.pop(k, None)
            else:
                os.environ[k] = v


AC_SHAPES = [(20, 36, 132), (5, 64, 256), (1, 9, 128), (3, 1, 4), (2, 50, 260), (9, 33, 516), (40, 8, 128),
             (6, 70, 388)]


@pytest.mark.parametrize("pts", [7, 13])
@pytest.mark.parametrize("shape", AC_SHAPES)
def test_k2ra_bitwise_equal_single_steps(lift, pts, shape):
    rng = np.random.default_rng(80)
    u0 = rng.uniform(-1, 1, size=shape).astype(np.float32)
    u1 = rng.uniform(-1, 1, size=shape).astype(np.float32)
    sp = ac_spec(shape, pts)
    n1, p1, _ = ac_run(lift, sp, u0, u1, 6, 2)
    n2, p2, plan = ac_run(lift, sp, u0, u1, 6, 4)
    assert plan.last_kernel == "k2ra_sweep"
    np.testing.assert_array_equal(n2, n1)
    np.testing.assert_array_equal(p2, p1)


@pytest.mark.parametrize("pts,shape_env", [(7, "4"), (7, "8"), (7, "6"), (13, "2"), (13, "3"), (13, "4")])
@pytest.mark.parametrize("zc", [("1", "0"), ("3", "1"), ("64", "0"), ("5", "2")])
def test_k2ra_shapes_and_chunks(lift, pts, shape_env, zc):
    shape = (17, 70, 260)
    rng = np.random.default_rng(81)
    u0 = rng.uniform(-1, 1, size=shape).astype(np.float32)
    u1 = rng.uniform(-1, 1, size=shape).astype(np.float32)
    sp = ac_spec(shape, pts)
    n1, p1, _ = ac_run(lift, sp, u0, u1, 4, 2)
    n2, p2, plan = ac_run(lift, sp, u0, u1, 4, 4, {"LIFT_K2RA_SHAPE": shape_env, "LIFT_K2RA_ZC": zc[0],
                                                   "LIFT_K2RA_ZC2": zc[1]})
    assert plan.last_kernel == "k2ra_sweep"
    np.testing.assert_array_equal(n2, n1)
    np.testing.assert_array_equal(p2, p1)


@pytest.mark.parametrize("pts", [7, 13])
def test_k2ra_vs_oracle_odd_steps(lift, pts):
    """7 steps = three K2RA passes + one single step, against the fp64 oracle
    (prev = cur initial condition as the BASELINE C5 recipe)."""
    shape = (14, 30, 132)
    u = np.random.default_rng(82).uniform(-1, 1, size=shape).astype(np.float32)
    sp = ac_spec(shape, pts)
    n2, p2, _ = ac_run(lift, sp, u, u, 7, 4)
    ref = orc.iterate(sp, [u, u], [], 7)
    assert np.max(np.abs(n2 - ref[1])) <= TOL10 * np.max(np.abs(ref[1]))
    assert np.max(np.abs(p2 - ref[0])) <= TOL10 * np.max(np.abs(ref[0]))
    n1, p1, _ = ac_run(lift, sp, u, u, 7, 2)
    np.testing.assert_array_equal(n2, n1)


def test_k2ra_time_block_1_and_two_buffers(lift):
    shape = (8, 20, 128)
    u = np.random.default_rng(83).uniform(-1, 1, size=shape).astype(np.float32)
    sp = ac_spec(shape, 7)
    _, _, plan = ac_run(lift, sp, u, u, 4, 4, tb=1)
    assert plan.last_kernel != "k2ra_sweep"
    _, _, plan = ac_run(lift, sp, u, u, 4, 2)
    assert plan.last_kernel != "k2ra_sweep"
    # AUTO (time block 0): two-step passes for the 7-point update only, on
    # grids that fill the GPU (>= 8 tiles of 128 x 32, >= 2048 (plane, tile) pairs)
    _, _, plan = ac_run(lift, sp, u, u, 4, 4, tb=0)
    assert plan.time_block == 1                              # too small for AUTO
    big = (64, 256, 1024)
    ub = np.random.default_rng(84).uniform(-1, 1, size=big).astype(np.float32)
    _, _, plan = ac_run(lift, ac_spec(big, 7), ub, ub, 2, 4, tb=0)
    assert plan.time_block == 2 and plan.last_kernel == "k2ra_sweep"
    _, _, plan = ac_run(lift, ac_spec(big, 13), ub, ub, 2, 4, tb=0)
    assert plan.time_block == 1 and plan.last_kernel != "k2ra_sweep"
    _, _, plan = ac_run(lift, ac_spec(shape, 13), u, u, 4, 4, tb=2)
    assert plan.time_block == 2 and plan.last_kernel == "k2ra_sweep"


def test_k2ra_acoustic13_1024_whole_grid(lift):
    """BASELINE C5b size (1024^3), 4 steps as two K2RA passes: bitwise equal to
    single steps over the whole grid (compared on the device)."""
    xs, sp = si.make_workload_inputs(si.workload("acoustic13_1024"))
    res = []
    for nbuf in (2, 4):
        plan = lift.Plan.from_spec(sp)
        plan.set_time_block(2)
        bufs = [torch.from_numpy(xs[0]).cuda(), torch.from_numpy(xs[1]).cuda()]
        bufs += [torch.empty_like(bufs[0]) for _ in range(nbuf - 2)]
        ri = plan.iterate(bufs, 4)
        torch.cuda.synchronize()
        res.append((bufs[ri], bufs[ri ^ 1], plan.last_kernel))
        del bufs
    assert res[1][2] == "k2ra_sweep"
    assert torch.equal(res[0][0], res[1][0]) and torch.equal(res[0][1], res[1][1])


# ------------------------------------------------------------------ K2CT ----
# Two Hotspot3D steps per launch for few-plane grids (whole-column tiles, the
# slid box with two halo rows/columns, X_{t+1} through registers into the
# same shared box; reindexing pads).

def hs_spec(extents, kind):
    kind = (kind,) * 3 if isinstance(kind, int) else tuple(kind)
    return si.StencilSpec(tuple(extents), (3, 3, 3), (1, 1, 1), (1, 1, 1), (1, 1, 1), kind, 0.0,
                          si.HOTSPOT3D, None, si.params_hotspot3d())


def hs_run(lift, sp, T, P, steps, tb, env=None):
    old = {}
    for k, v in (env or {}).items():
        old[k] = os.environ.get(k)
        os.environ[k] = v
    try:
        plan = lift.Plan.from_spec(sp)
        plan.set_time_block(tb)
        a = torch.from_numpy(T.copy()).cuda()
        b = torch.empty_like(a)
        pw = torch.from_numpy(P).cuda()
        ri = plan.iterate([a, b], steps, aux=[pw])
        torch.cuda.synchronize()
        return (a, b)[ri].cpu().numpy(), plan
    finally:
        for k, v in old.items():
            if v is None:
                os.environ.pop(k, None)
            else:
                os.environ[k] = v


HS_SHAPES = [(8, 64, 256), (8, 37, 260), (1, 9, 128), (2, 5, 132), (3, 1, 4), (16, 23, 388), (5, 70, 128),
             (8, 2, 516)]


@pytest.mark.parametrize("kind", [CLAMP, MIRROR, REFLECT, (CLAMP, REFLECT, MIRROR)])
@pytest.mark.parametrize("shape", HS_SHAPES)
def test_k2ct_bitwise_equal_single_steps(lift, kind, shape):
    rng = np.random.default_rng(90)
    T = rng.uniform(300, 350, size=shape).astype(np.float32)
    P = rng.uniform(0, 1e-2, size=shape).astype(np.float32)
    sp = hs_spec(shape, kind)
    y1, _ = hs_run(lift, sp, T, P, 6, 1)
    y2, plan = hs_run(lift, sp, T, P, 6, 2)
    assert plan.time_block == 2 and plan.last_kernel == "k2ct_column"
    np.testing.assert_array_equal(y2, y1)


@pytest.mark.parametrize("ty", ["4", "5"])
def test_k2ct_tile_heights_and_odd_steps(lift, ty):
    shape = (8, 41, 260)
    rng = np.random.default_rng(91)
    T = rng.uniform(300, 350, size=shape).astype(np.float32)
    P = rng.uniform(0, 1e-2, size=shape).astype(np.float32)
    sp = hs_spec(shape, CLAMP)
    y1, _ = hs_run(lift, sp, T, P, 7, 1)
    y2, plan = hs_run(lift, sp, T, P, 7, 2, {"LIFT_K2CT_TY": ty})
    np.testing.assert_array_equal(y2, y1)
    ref = orc.iterate(sp, [T], [P], 7)[0]
    assert np.max(np.abs(y2 - ref) / np.abs(ref)) <= TOL10


def test_k2ct_hotspot3d_8x512x512_whole_grid(lift):
    """BASELINE C4a size, 10 steps as 5 K2CT launches: bitwise equal to single steps."""
    xs, sp = si.make_workload_inputs(si.workload("hotspot3d_8x512x512_x100"))
    y1, _ = hs_run(lift, sp, xs[0], xs[1], 10, 1)
    y2, plan = hs_run(lift, sp, xs[0], xs[1], 10, 2)
    assert plan.last_kernel == "k2ct_column"
    _, plan = hs_run(lift, sp, xs[0], xs[1], 2, 0)
    assert plan.time_block == 1 and plan.last_kernel == "k2c_column"     # AUTO: single steps
    assert np.array_equal(y2, y1)


# ------------------------------------------------------- run_host_batch ----
@pytest.mark.parametrize("case", ["j3d7", "acoustic7", "hotspot"])
def test_run_host_batch_matches_run_host(lift, case):
    """stencil_run_host_batch: every job's output equals stencil_run_host's
    (bitwise), with jobs of different inputs, more jobs than workspace slots."""
    rng = np.random.default_rng(130)
    if case == "j3d7":
        shape = (20, 40, 136)
        sp = spec(shape, CLAMP)
        jobs = [[rng.uniform(0.5, 1.5, size=shape).astype(np.float32)] for _ in range(5)]
        aux = ()
    elif case == "acoustic7":
        shape = (12, 30, 132)
        sp = ac_spec(shape, 7)
        jobs = [[rng.uniform(-1, 1, size=shape).astype(np.float32) for _ in range(2)] for _ in range(5)]
        aux = ()
    else:
        shape = (8, 30, 128)
        sp = hs_spec(shape, CLAMP)
        jobs = [[rng.uniform(300, 350, size=shape).astype(np.float32)] for _ in range(5)]
        aux = [[rng.uniform(0, 1e-2, size=shape).astype(np.float32)] for _ in range(5)]
    plan = lift.Plan.from_spec(sp)
    outs = plan.run_host_batch(jobs, 6, aux)
    for j in range(5):
        ref = plan.run_host(jobs[j], n_steps=6, host_aux=aux[j] if aux else ())
        np.testing.assert_array_equal(outs[j], ref)
