"""Every point at BASELINE.json's full sizes (no sampling).

Tiled must equal untiled everywhere (overlapped tiling preserves the
stencil's semantics).  Two whole-grid checks, in the
launch configuration bench.py times (AUTO kernel selection):

  * single sweeps against the fp64 oracle at EVERY output point: the oracle
    computes the grid in blocks of output planes (oracle.apply_planes: the
    same definition restricted to a block, each block padded from its own
    input planes), spread over the host cores by a fork-based process pool
    (the workers only run numpy on the inherited arrays); tolerance 1e-5 per
    point (north_star, A22);
  * the production kernels against K0 (the generic one-thread-per-output
    kernel, STENCIL_VARIANT_GENERIC) bitwise over the whole grid, for single
    sweeps and for 10-step iterates (every kernel family evaluates each point
    with the same operation sequence, A12).
"""
import multiprocessing as mp
import os

import numpy as np
import pytest
import torch

import stencil_inputs as si
from oracle import stencil_oracle as orc

pytestmark = [pytest.mark.gpu, pytest.mark.slow,
              # the pool forks a process that has CUDA threads; the children run numpy only
              pytest.mark.filterwarnings("ignore:This process .* is multi-threaded:DeprecationWarning")]

_JOB = {}


@pytest.fixture(scope="module")
def lift():
    import __graft_entry__
    __graft_entry__.build()
    import paper_conf_cgo_hagedornssgd18_b200 as m
    torch.cuda.set_device(0)
    return m


def _block_err(block):
    spec, xs, g = _JOB["spec"], _JOB["xs"], _JOB["g"]
    z0, z1 = block
    Y, A = orc.apply_planes(spec, xs, z0, z1)
    return orc.max_rel_err(g[z0:z1], Y, A)


def oracle_full_grid_err(spec, xs, g):
    """max over every output point of |g - o| / max(|o|, A) (reading A22)."""
    n0 = spec.out_extents()[0]
    per_plane = int(np.prod(spec.out_extents()[1:]))
    chunk = max(1, (4 << 20) // per_plane)
    blocks = [(z, min(z + chunk, n0)) for z in range(0, n0, chunk)]
    _JOB.update(spec=spec, xs=xs, g=g)
    try:
        procs = max(1, min(os.cpu_count() or 1, 16, len(blocks)))
        with mp.get_context("fork").Pool(procs) as pool:
            errs = pool.map(_block_err, blocks, chunksize=1)
    finally:
        _JOB.clear()
    return max(errs)


def run(lift, spec, xs, steps=1, variant=None):
    """The plan's output (1 step: apply; n: iterate) as a device tensor."""
    plan = lift.Plan.from_spec(spec)
    if variant is not None:
        plan.set_variant(variant)
    dev = [torch.from_numpy(x).cuda() for x in xs]
    if steps == 1:
        y = plan.apply(*dev)
        torch.cuda.synchronize()
        return y, plan
    if spec.op == si.ACOUSTIC:
        st, aux = dev, []
    else:
        st, aux = [dev[0], torch.empty_like(dev[0])], dev[1:]
    ri = plan.iterate(st, steps, aux)
    torch.cuda.synchronize()
    return st[ri], plan


SWEEPS = ["j2d5_256_clamp", "gauss5_8192_mirror", "j3d7_512_clamp", "hotspot3d_8x512x512", "srad1_4096",
          "srad2_4096", "acoustic7_1024", "acoustic13_1024", "t1_stencil2d_4098", "t1_srad1_504x458",
          "t1_hotspot2d_8192", "t1_gradient_4096", "t1_jacobi2d9_8192", "t1_poisson19_512", "t1_heat7_512",
          "t1_jacobi3d13_512", "t1_acoustic_404x512x512"]


@pytest.mark.parametrize("name", SWEEPS)
def test_single_sweep_every_point_vs_oracle(lift, name):
    xs, spec = si.make_workload_inputs(si.workload(name))
    y, plan = run(lift, spec, xs)
    assert plan.last_variant != 0, "full-size config must run on a tiled kernel"
    g = y.cpu().numpy()
    del y
    err = oracle_full_grid_err(spec, xs, g)
    assert err <= 1e-5, f"{name}: max rel err {err:.3e} over {g.size} points"


def test_srad_iteration_every_point_vs_oracle(lift):
    xs, spec = si.make_workload_inputs(si.workload("srad_iter_4096"))
    y, plan = run(lift, spec, xs)
    assert plan.last_variant == 1
    Y, A = orc.apply(spec, xs)          # q0 is a whole-image statistic: one block
    assert orc.max_rel_err(y.cpu().numpy(), Y, A) <= 1e-5


@pytest.mark.parametrize("name,steps", [("gauss5_8192_mirror", 1), ("j3d7_512_clamp", 1), ("j3d7_512_clamp", 10),
                                        ("acoustic7_1024", 1), ("acoustic7_1024", 10), ("acoustic13_1024", 1),
                                        ("acoustic13_1024", 10), ("hotspot3d_8x512x512", 10),
                                        ("srad_iter_4096", 1), ("srad1_4096", 1), ("srad2_4096", 1),
                                        ("t1_stencil2d_4098", 1), ("t1_hotspot2d_8192", 1), ("t1_gradient_4096", 1),
                                        ("t1_jacobi2d9_8192", 1), ("t1_poisson19_512", 1), ("t1_heat7_512", 10),
                                        ("t1_jacobi3d13_512", 10), ("t1_acoustic_404x512x512", 10)])
def test_production_equals_generic_whole_grid(lift, name, steps):
    xs, spec = si.make_workload_inputs(si.workload(name))
    y, plan = run(lift, spec, xs, steps)
    assert plan.last_variant != 0
    y0, plan0 = run(lift, spec, xs, steps, variant="generic")
    assert plan0.last_variant == 0
    assert torch.equal(y, y0), (f"{name} x{steps}: {int((y != y0).sum())} of {y.numel()} points differ "
                                f"from K0")
