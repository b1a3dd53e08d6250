"""Seeded synthetic workloads shared by the oracle side and the CUDA side.

This module holds NO stencil arithmetic.  It only says *what* is computed
(extents, pad/slide arguments, boundary kinds, weights, op constants) and
draws the seeded fp32 input grids.  Both ``oracle/`` (test infrastructure) and
the CUDA path's tests/bench import it; neither imports the other.

Workload recipe:
  * grids are contiguous fp32, row-major, extents slowest-first (PAPER.md
    P:336-337, ``[[T]_m]_n`` has n outermost);
  * values come from ``numpy.random.default_rng(seed).random(shape, float32)``
    (PCG64, U[0,1)) and are mapped affinely in fp32 per workload;
  * seeds 1001..1007 follow SURVEY.md §8(d).

Weights/constants are the readings A13, A14, A16, A18, A19, A20 of DESIGN.md
(the paper prints none: Table 1, gives only dims/points/sizes).
"""
from __future__ import annotations

from dataclasses import dataclass
from typing import List, Optional, Sequence, Tuple

import numpy as np

# Boundary kinds — numeric values are the C-ABI enum ``stencil_pad``.
CLAMP, MIRROR, WRAP, CONSTANT, REFLECT, DAMPEN = 0, 1, 2, 3, 4, 5
KIND_NAMES = {CLAMP: "clamp", MIRROR: "mirror", WRAP: "wrap",
              CONSTANT: "constant", REFLECT: "reflect", DAMPEN: "dampen"}

# Ops — numeric values are the C-ABI enum ``stencil_op``.
WEIGHTED, HOTSPOT3D, SRAD1, SRAD2, ACOUSTIC, HOTSPOT2D, GRADIENT, SRAD = 0, 1, 2, 3, 4, 5, 6, 7
OP_NAMES = {WEIGHTED: "weighted", HOTSPOT3D: "hotspot3d", SRAD1: "srad1",
            SRAD2: "srad2", ACOUSTIC: "acoustic", HOTSPOT2D: "hotspot2d", GRADIENT: "gradient",
            SRAD: "srad"}

# Number of input grids per op (zip arity).
N_INPUTS = {WEIGHTED: 1, HOTSPOT3D: 2, SRAD1: 1, SRAD2: 2, ACOUSTIC: 2, HOTSPOT2D: 2, GRADIENT: 1, SRAD: 1}


@dataclass
class StencilSpec:
    """Arguments of ``map_n(f, slide_n(size, step, pad_n(l, r, h, input)))``
     plus the op id/constants of the map function."""
    extents: Tuple[int, ...]            # n_d, slowest first
    size: Tuple[int, ...]               # slide size per dim
    step: Tuple[int, ...]               # slide step per dim
    pad_lo: Tuple[int, ...]             # pad l per dim
    pad_hi: Tuple[int, ...]             # pad r per dim
    kind: Tuple[int, ...]               # boundary function h per dim
    pad_value: float = 0.0              # value for CONSTANT
    op: int = WEIGHTED
    weights: Optional[np.ndarray] = None    # float32, shape == size (WEIGHTED)
    params: Tuple[float, ...] = ()          # float32 op constants
    pad_decay: float = 1.0                  # DAMPEN dimensions: decay per cell of distance (reading A29)

    @property
    def ndim(self) -> int:
        return len(self.extents)

    def out_extents(self) -> Tuple[int, ...]:
        """o_d = floor((n_d + l_d + r_d - size_d) / step_d) + 1 (A6)."""
        return tuple((n + l + r - s) // st + 1 for n, l, r, s, st in
                     zip(self.extents, self.pad_lo, self.pad_hi, self.size, self.step))


def f32(x) -> np.ndarray:
    return np.asarray(x, dtype=np.float32)


# --------------------------------------------------------------------------
# Weights (A13, A14). Row-major over the neighbourhood, slowest dim
# first, offset -r first.
# --------------------------------------------------------------------------
def weights_j2d5() -> np.ndarray:
    """Jacobi 2D 5-point (A13): N=.10 W=.15 C=.45 E=.10 S=.20, asymmetric."""
    return f32([[0.0, 0.10, 0.0],
                [0.15, 0.45, 0.10],
                [0.0, 0.20, 0.0]])


def weights_j2d9() -> np.ndarray:
    """Jacobi 2D 9-point (box), normalised, asymmetric (NEXT-1 shape)."""
    w = np.array([[0.05, 0.10, 0.06],
                  [0.12, 0.30, 0.08],
                  [0.07, 0.14, 0.08]], dtype=np.float64)
    return f32(w)


def weights_j3d7() -> np.ndarray:
    """Jacobi 3D 7-point star (A13): C=.40, z-1=.05, z+1=.15, y+-1=.10, x-1=.08, x+1=.12."""
    w = np.zeros((3, 3, 3), np.float32)
    w[1, 1, 1] = 0.40
    w[0, 1, 1] = 0.05
    w[2, 1, 1] = 0.15
    w[1, 0, 1] = 0.10
    w[1, 2, 1] = 0.10
    w[1, 1, 0] = 0.08
    w[1, 1, 2] = 0.12
    return w


def weights_j3d13() -> np.ndarray:
    """Jacobi 3D 13-point star, radius 2 (A13): C=.28, +-1 taps .08, +-2 taps .04."""
    w = np.zeros((5, 5, 5), np.float32)
    w[2, 2, 2] = 0.28
    for d in range(3):
        for off, val in ((1, 0.08), (2, 0.04)):
            for sgn in (-1, 1):
                idx = [2, 2, 2]
                idx[d] = 2 + sgn * off
                w[tuple(idx)] = val
    return w


def weights_gauss5() -> np.ndarray:
    """Gaussian 5x5 binomial [1,4,6,4,1] (x) [1,4,6,4,1] / 256 (A14); exact in fp32."""
    b = np.array([1, 4, 6, 4, 1], np.float64)
    return f32(np.outer(b, b) / 256.0)


def weights_laplacian(ndim: int) -> np.ndarray:
    """Discrete Laplacian (A13, tests only): centre -2*ndim, faces +1."""
    w = np.zeros((3,) * ndim, np.float32)
    c = (1,) * ndim
    w[c] = -2.0 * ndim
    for d in range(ndim):
        for s in (0, 2):
            idx = list(c)
            idx[d] = s
            w[tuple(idx)] = 1.0
    return w


# --------------------------------------------------------------------------
# Op constants (A16, A18, A19, A20)
# --------------------------------------------------------------------------
def params_hotspot3d() -> Tuple[float, ...]:
    """Rodinia v3.1 hotspot3D constants for a (8, 512, 512) chip (A16).
    Order: cc, cn, cs, ce, cw, ct, cb, sdc, amb."""
    ce = cw = cn = cs = 0.0341333
    ct = cb = 5.33333e-4
    cc = 1.0 - (2 * ce + 2 * cn + 3 * ct)
    sdc = 0.341333
    amb = 80.0
    return tuple(float(np.float32(v)) for v in (cc, cn, cs, ce, cw, ct, cb, sdc, amb))


def params_hotspot2d(rows: int, cols: int) -> Tuple[float, ...]:
    """Rodinia v3.1 hotspot constants for a rows x cols chip (A26).
    Order: step/Cap, 1/Rx, 1/Ry, 1/Rz, amb."""
    t_chip, chip_h, chip_w = 0.0005, 0.016, 0.016
    k_si, spec_heat_si, factor_chip, max_pd, precision, amb = 100.0, 1.75e6, 0.5, 3.0e6, 0.001, 80.0
    gh, gw = chip_h / rows, chip_w / cols
    cap = factor_chip * spec_heat_si * t_chip * gw * gh
    rx = gw / (2.0 * k_si * t_chip * gh)
    ry = gh / (2.0 * k_si * t_chip * gw)
    rz = t_chip / (k_si * gh * gw)
    max_slope = max_pd / (factor_chip * t_chip * spec_heat_si)
    step = precision / max_slope
    return tuple(float(np.float32(v)) for v in (step / cap, 1.0 / rx, 1.0 / ry, 1.0 / rz, amb))


def params_gradient() -> Tuple[float, ...]:
    """eps of the 2D gradient (A25)."""
    return (float(np.float32(1e-4)),)


def weights_heat7() -> np.ndarray:
    """Heat 3D 7-point ([35], A13): u + 0.125 * (discrete Laplacian)."""
    w = np.zeros((3, 3, 3), np.float32)
    w[1, 1, 1] = 1.0 - 6 * 0.125
    for d in range(3):
        for sgn in (0, 2):
            idx = [1, 1, 1]
            idx[d] = sgn
            w[tuple(idx)] = 0.125
    return w


def weights_poisson19() -> np.ndarray:
    """Poisson 3D 19-point ([35], A13): centre 1/4, 6 faces 1/16, 12 edges 1/32 (normalised, dyadic)."""
    w = np.zeros((3, 3, 3), np.float32)
    for k in np.ndindex(3, 3, 3):
        nax = sum(1 for v in k if v != 1)
        w[k] = {0: 0.25, 1: 1.0 / 16, 2: 1.0 / 32}.get(nax, 0.0)
    return w


def params_srad1(q0sqr: float) -> Tuple[float, ...]:
    return (float(np.float32(q0sqr)),)


def params_srad2(lam: float = 0.5) -> Tuple[float, ...]:
    return (float(np.float32(lam)),)


def params_acoustic(points: int) -> Tuple[float, ...]:
    """(lambda^2, loss1, loss2) (A19/A20): zeta = 0.1, loss1 = 1/(1+zeta),
    loss2 = 1 - zeta; lambda^2 = 0.25 (7-point) or 0.15 (13-point)."""
    zeta = 0.1
    l2 = 0.25 if points == 7 else 0.15
    return tuple(float(np.float32(v)) for v in (l2, 1.0 / (1.0 + zeta), 1.0 - zeta))


def srad_q0sqr(image: np.ndarray) -> float:
    """Rodinia's q0sqr = var/mean^2 of the image (A18), computed once on the
    host in fp64 from the input and passed to both sides as an fp32 param.
    This is a workload parameter (a statistic of the input), not stencil work."""
    x = image.astype(np.float64)
    m = x.mean()
    return float(np.float32(x.var() / (m * m)))


# --------------------------------------------------------------------------
# Seeded grids
# --------------------------------------------------------------------------
def uniform(shape: Sequence[int], seed: int, lo: float = 0.0, hi: float = 1.0) -> np.ndarray:
    """U[lo, hi) fp32 from PCG64(seed); the affine map is done in fp32."""
    rng = np.random.default_rng(seed)
    u = rng.random(tuple(shape), dtype=np.float32)
    if lo != 0.0 or hi != 1.0:
        u *= np.float32(hi - lo)
        u += np.float32(lo)
    return u


@dataclass
class Workload:
    """One named configuration: a spec plus how to draw its inputs."""
    name: str
    spec: StencilSpec
    seeds: Tuple[int, ...]
    ranges: Tuple[Tuple[float, float], ...]
    steps: int = 1                      # time steps (iterate), 1 = single sweep
    transform: Tuple[str, ...] = ()     # per-input post-transform ('exp' for SRAD)
    note: str = ""

    def make_inputs(self) -> List[np.ndarray]:
        xs = []
        for i, (seed, (lo, hi)) in enumerate(zip(self.seeds, self.ranges)):
            x = uniform(self.spec.extents, seed, lo, hi)
            if i < len(self.transform) and self.transform[i] == "exp":
                x = np.exp(x).astype(np.float32)
            xs.append(x)
        return xs


def _spec(extents, size, op=WEIGHTED, weights=None, params=(), kind=CLAMP,
          pad=None, step=None, pad_value=0.0) -> StencilSpec:
    nd = len(extents)
    size = tuple(size) if isinstance(size, (tuple, list)) else (size,) * nd
    r = tuple(s // 2 for s in size) if pad is None else (
        tuple(pad) if isinstance(pad, (tuple, list)) else (pad,) * nd)
    kind = tuple(kind) if isinstance(kind, (tuple, list)) else (kind,) * nd
    step = (1,) * nd if step is None else tuple(step)
    return StencilSpec(tuple(extents), size, step, r, r, kind, pad_value, op,
                       None if weights is None else f32(weights), tuple(params))


def workload(name: str, scale: Optional[Tuple[int, ...]] = None) -> Workload:
    """Named workloads of BASELINE.json ``configs`` (C1..C5) and the
    paper-shaped extras.  ``scale`` overrides the extents (parity-sized runs)."""
    W = _WORKLOADS[name]
    w = W()
    if scale is not None:
        w.spec.extents = tuple(scale)
    return w


def _c1():
    return Workload("j2d5_256_clamp", _spec((256, 256), 3, weights=weights_j2d5()),
                    (1001,), ((0.5, 1.5),), 1, note="C1: Jacobi 2D 5-point, clamp, single sweep")


def _c2():
    return Workload("gauss5_8192_mirror", _spec((8192, 8192), 5, weights=weights_gauss5(), kind=MIRROR),
                    (1002,), ((0.5, 1.5),), 1, note="C2: Gaussian 5x5, mirror (symmetric), single sweep")


def _c3():
    return Workload("j3d7_512_clamp", _spec((512, 512, 512), 3, weights=weights_j3d7()),
                    (1003,), ((0.5, 1.5),), 100, note="C3: Jacobi 3D 7-point, clamp, 100 time steps")


def _c4a():
    return Workload("hotspot3d_8x512x512", _spec((8, 512, 512), 3, op=HOTSPOT3D, params=params_hotspot3d()),
                    (1004, 1005), ((300.0, 350.0), (0.0, 1e-2)), 1, note="C4a: Rodinia Hotspot3D, clamp")


def _c4a100():
    return Workload("hotspot3d_8x512x512_x100", _spec((8, 512, 512), 3, op=HOTSPOT3D, params=params_hotspot3d()),
                    (1004, 1005), ((300.0, 350.0), (0.0, 1e-2)), 100,
                    note="C4a iterated (SURVEY §8(d)): Rodinia Hotspot3D, clamp, 100 time steps")


def _c4b1():
    return Workload("srad1_4096", _spec((4096, 4096), 3, op=SRAD1), (1006,), ((0.0, 1.0),), 1,
                    transform=("exp",), note="C4b: Rodinia SRAD1 (I -> c), clamp; q0sqr from the input")


def _c4b2():
    return Workload("srad2_4096", _spec((4096, 4096), 3, op=SRAD2, params=params_srad2()),
                    (1008, 1006), ((0.0, 1.0), (0.0, 1.0)), 1, transform=("", "exp"),
                    note="C4b: Rodinia SRAD2 ((c, I) -> I'), clamp")


def _c5a():
    return Workload("acoustic7_1024", _spec((1024, 1024, 1024), 3, op=ACOUSTIC, params=params_acoustic(7),
                                           kind=CONSTANT, pad_value=0.0),
                    (1007, 1007), ((-1.0, 1.0), (-1.0, 1.0)), 100,
                    note="C5a: Acoustic 7-point (Listing 3), zero pad, prev = cur")


def _c5b():
    return Workload("acoustic13_1024", _spec((1024, 1024, 1024), 5, op=ACOUSTIC, params=params_acoustic(13),
                                            kind=CONSTANT, pad_value=0.0),
                    (1007, 1007), ((-1.0, 1.0), (-1.0, 1.0)), 100,
                    note="C5b: Acoustic 13-point (A20 extrapolation), zero pad, prev = cur")


# Table 1 shapes through the same ABI ("paper-shaped sweep", NEXT-1)
def _t1(name, extents, size, op=WEIGHTED, weights=None, params=(), kind=CLAMP, seeds=(2001,),
        ranges=((0.5, 1.5),), transform=(), note=""):
    return lambda: Workload(name, _spec(extents, size, op=op, weights=weights, params=params, kind=kind),
                            seeds, ranges, 1, transform, note)


_TABLE1 = {
    "t1_stencil2d_4098": _t1("t1_stencil2d_4098", (4098, 4098), 3, weights=weights_j2d9(),
                             note="SHOC Stencil2D 9-point (weights: A13 J2D9 reading)"),
    "t1_srad1_504x458": _t1("t1_srad1_504x458", (504, 458), 3, op=SRAD1, transform=("exp",), ranges=((0.0, 1.0),),
                            note="Rodinia SRAD1 at the paper's size"),
    "t1_hotspot2d_8192": _t1("t1_hotspot2d_8192", (8192, 8192), 3, op=HOTSPOT2D,
                             params=params_hotspot2d(8192, 8192), seeds=(2002, 2003),
                             ranges=((300.0, 350.0), (0.0, 1e-2)), note="Rodinia Hotspot2D (A26)"),
    "t1_acoustic_404x512x512": _t1("t1_acoustic_404x512x512", (404, 512, 512), 3, op=ACOUSTIC,
                                   params=params_acoustic(7), kind=CONSTANT, seeds=(2004, 2004),
                                   ranges=((-1.0, 1.0), (-1.0, 1.0)), note="Acoustic at the paper's size"),
    "t1_gaussian_4096": _t1("t1_gaussian_4096", (4096, 4096), 5, weights=weights_gauss5(), kind=MIRROR),
    "t1_gradient_4096": _t1("t1_gradient_4096", (4096, 4096), 3, op=GRADIENT, params=params_gradient(),
                            note="Rawat 2D gradient (A25)"),
    "t1_gradient_8192": _t1("t1_gradient_8192", (8192, 8192), 3, op=GRADIENT, params=params_gradient()),
    "t1_jacobi2d5_8192": _t1("t1_jacobi2d5_8192", (8192, 8192), 3, weights=weights_j2d5()),
    "t1_jacobi2d9_8192": _t1("t1_jacobi2d9_8192", (8192, 8192), 3, weights=weights_j2d9()),
    "t1_jacobi3d7_256": _t1("t1_jacobi3d7_256", (256, 256, 256), 3, weights=weights_j3d7()),
    "t1_jacobi3d13_512": _t1("t1_jacobi3d13_512", (512, 512, 512), 5, weights=weights_j3d13()),
    "t1_poisson19_512": _t1("t1_poisson19_512", (512, 512, 512), 3, weights=weights_poisson19(),
                            note="Poisson 19-point (A13 reading)"),
    "t1_heat7_512": _t1("t1_heat7_512", (512, 512, 512), 3, weights=weights_heat7()),
}

_WORKLOADS = {
    "j2d5_256_clamp": _c1,
    "gauss5_8192_mirror": _c2,
    "j3d7_512_clamp": _c3,
    "hotspot3d_8x512x512": _c4a,
    "srad1_4096": _c4b1,
    "srad2_4096": _c4b2,
    "acoustic7_1024": _c5a,
    "acoustic13_1024": _c5b,
}

def _srad_iter():
    return Workload("srad_iter_4096", _spec((4096, 4096), 3, op=SRAD, params=params_srad2()), (1006,), ((0.0, 1.0),),
                    20, transform=("exp",),
                    note="NEXT-2: full SRAD iterations (q0 reduction + fused SRAD1/SRAD2), clamp, 20 iterations")


_WORKLOADS["srad_iter_4096"] = _srad_iter
_WORKLOADS["hotspot3d_8x512x512_x100"] = _c4a100
_WORKLOADS.update(_TABLE1)
WORKLOAD_NAMES = tuple(_WORKLOADS)
TABLE1_NAMES = tuple(_TABLE1)


def make_workload_inputs(w: Workload) -> Tuple[List[np.ndarray], StencilSpec]:
    """Draw inputs; fills input-derived params (SRAD1 q0sqr) into the spec."""
    xs = w.make_inputs()
    spec = w.spec
    if spec.op == SRAD1:
        spec.params = params_srad1(srad_q0sqr(xs[0]))
    return xs, spec


# ---- counter-based grids for sizes too large to draw on the host ----------
# value(i) = 1 + (h(i) >> 9) * 2^-23 in [1, 2), exact in fp32, where h is a
# 32-bit integer hash of the linear index i.  The device side evaluates the
# same integer formula with torch int64 ops (hash_grid_torch); the oracle side
# reads single points through HashGrid[...] (no arithmetic of the method).
_M32 = 0xFFFFFFFF


def _hash32(i: int, seed: int) -> int:
    h = (i * 2654435761 + seed) & _M32
    h ^= h >> 15
    h = (h * 2246822519) & _M32
    h ^= h >> 13
    return h


class HashGrid:
    """Read-only fp32 grid of the given extents whose element at linear index i
    is ``1 + (hash32(i, seed) >> 9) * 2**-23``; indexable by index tuples."""

    def __init__(self, extents: Sequence[int], seed: int):
        self.shape = tuple(int(e) for e in extents)
        self.seed = int(seed)
        self.strides = tuple(int(np.prod(self.shape[d + 1:])) for d in range(len(self.shape)))

    def __getitem__(self, idx) -> np.float32:
        lin = sum(int(i) * s for i, s in zip(idx, self.strides))
        return np.float32(1.0 + (_hash32(lin, self.seed) >> 9) * 2.0 ** -23)


def hash_grid_torch(extents: Sequence[int], seed: int, device, chunk: int = 1 << 26):
    """The HashGrid values materialised on ``device`` (torch int64 arithmetic
    in chunks; int64 products wrap mod 2^64, so the low 32 bits are exact)."""
    import torch
    n = int(np.prod(extents))
    out = torch.empty(n, dtype=torch.float32, device=device)
    for a in range(0, n, chunk):
        b = min(n, a + chunk)
        h = (torch.arange(a, b, dtype=torch.int64, device=device) * 2654435761 + seed) & _M32
        h ^= h >> 15
        h = (h * 2246822519) & _M32
        h ^= h >> 13
        out[a:b] = ((h >> 9).to(torch.float32) * 2.0 ** -23) + 1.0
    return out.view(*extents)
