"""CPU fp64 oracle for the Lift stencil hot path — TEST INFRASTRUCTURE ONLY.

Only ``tests/``, ``__graft_entry__.smoke()`` and ``bench.py``'s
``cpu_baseline`` / ``--impl reference`` legs may import this module.  The
product path (``paper_conf_cgo_hagedornssgd18_b200``) never imports it and
shares no code with it.

What it computes is the paper's problem statement written out literally
(§3.4):

    map_n(f, slide_n(size, step, pad_n(l, r, h, input)))

in the paper's order: (1) ``pad_n`` materialises the padded grid, one
dimension at a time, outer dimension first; (2) ``slide_n`` takes
the window ``W_o[k] = P[o*step + k]`` for every output index ``o``
(tap k of a window is padded index ``o*step + k``,
reading A7); (3) ``map`` applies the neighbourhood function f to every window
(P:491-497), with any extra grids zipped point-wise (``zip``; Listing 3
P:649-662); (4) ``iterate`` feeds outputs back.
Arithmetic is fp64; fp32 inputs and fp32-rounded constants are promoted
exactly (reading A23).  numpy is used for array indexing and elementwise fp64
arithmetic only; there is no blocking, fusion or reordering beyond the
definition.

Pins (tests/test_oracle_*.py): brute force vs ``numpy.pad`` modes and
``sliding_window_view``; the paper's printed pad2 and slide2
 examples; Listing 1; weighted map vs
``torch.nn.functional.conv{1,2,3}d`` in fp64; invariants (constant field,
linear field under the Laplacian, Gaussian separability, wrap translation
equivariance, mirror symmetry, linearity).

The non-linear point functions are EXTERNAL READINGS (the paper prints no
formula or values, A16/A18/A19/A25/A26): Hotspot3D, Hotspot2D,
SRAD1/SRAD2, Gradient and the Acoustic constants.  Given the reading, each is
pinned independently of this file: Hotspot3D/2D, SRAD2 and Gradient by
independently written scalar Rodinia-style loops; SRAD1 by hand-derived closed
forms (isolated spike q = eps^2, face neighbour 7eps^2/(16(1+eps/4)^2), ramp
q = b^2/I^2, c = q0(1+q0)/(q0^2+q)); q0^2 by closed-form images; the
Acoustic grid roles by the leapfrog identity u' = 2u^n - u^{n-1} on a linear
u^n with random u^{n-1} and by the locality of each grid; K by brute force.
What stays unpinned is only whether the readings are the paper's intent.
"""
from __future__ import annotations

from typing import Callable, List, Sequence, Tuple

import numpy as np

CLAMP, MIRROR, WRAP, CONSTANT, REFLECT, DAMPEN = 0, 1, 2, 3, 4, 5
WEIGHTED, HOTSPOT3D, SRAD1, SRAD2, ACOUSTIC, HOTSPOT2D, GRADIENT, SRAD = 0, 1, 2, 3, 4, 5, 6, 7


# ---------------------------------------------------------------------------
# Index functions h(i, n) of the reindexing pad
# ---------------------------------------------------------------------------
def h_clamp(i, n):
    """clamp(i, n) = (i < 0) ? 0 : ((i >= n) ? n-1 : i)."""
    i = np.asarray(i)
    return np.where(i < 0, 0, np.where(i >= n, n - 1, i))


def h_mirror(i, n):
    """Mirror, symmetric with the edge repeated (reading A2; P:457 says only
    "similarly defined"): i<0 -> -1-i; then i mod 2n; then i>=n -> 2n-1-i."""
    i = np.asarray(i)
    i = np.where(i < 0, -1 - i, i)
    i = np.mod(i, 2 * n)
    return np.where(i >= n, 2 * n - 1 - i, i)


def h_wrap(i, n):
    """Wrap (reading A3): ((i mod n) + n) mod n."""
    i = np.asarray(i)
    return np.mod(np.mod(i, n) + n, n)


def h_reflect(i, n):
    """Reflect, edge not repeated (reading A2, exported as a separate kind):
    period 2n-2; n == 1 maps everything to 0."""
    i = np.asarray(i)
    if n == 1:
        return np.zeros_like(i)
    p = 2 * n - 2
    i = np.mod(i, p)
    return np.where(i >= n, p - i, i)


H = {CLAMP: h_clamp, MIRROR: h_mirror, WRAP: h_wrap, REFLECT: h_reflect}


# ---------------------------------------------------------------------------
# pad and pad_n
# ---------------------------------------------------------------------------
def dampen_distance(i, n):
    """Distance of unpadded index i outside [0, n): -i left, i-n+1 right, 0 inside."""
    i = np.asarray(i)
    return np.where(i < 0, -i, np.where(i >= n, i - n + 1, 0))


def pad1(x: np.ndarray, axis: int, l: int, r: int, kind: int, value: float = 0.0,
         decay: float = 1.0) -> np.ndarray:
    """1D pad applied along ``axis``: type [T]_n -> [T]_{l+n+r}.

    Reindexing variant: padded index j in [0, l+n+r) reads x[h(j - l, n)]
    (h receives i - l in [-l, n+r), reading A1).  Value variant:
    positions outside [l, l+n) hold ``value`` (CONSTANT, reading A4).
    DAMPEN ("dampening boundary conditions where the out-of-bound value
    decreases with the distance to the boundary"; reading A29):
    the cell at distance d >= 1 outside the array holds the nearest element
    times decay**d."""
    n = x.shape[axis]
    if kind == DAMPEN:
        i = np.arange(-l, n + r)
        out = np.take(np.asarray(x, np.float64), h_clamp(i, n), axis=axis)
        shape = [1] * out.ndim
        shape[axis] = l + n + r
        return out * (np.float64(decay) ** dampen_distance(i, n)).reshape(shape)
    if kind == CONSTANT:
        shape = list(x.shape)
        shape[axis] = l + n + r
        out = np.full(shape, np.float64(value), dtype=np.float64)
        sl = [slice(None)] * x.ndim
        sl[axis] = slice(l, l + n)
        out[tuple(sl)] = x
        return out
    idx = H[kind](np.arange(-l, n + r), n)
    return np.take(x, idx, axis=axis).astype(np.float64, copy=False)


def pad_n(x: np.ndarray, pad_lo: Sequence[int], pad_hi: Sequence[int],
          kind: Sequence[int], value: float = 0.0, decay: float = 1.0) -> np.ndarray:
    """pad_n(l, r, h, input) = map_{n-1}(pad(l, r, h), pad_{n-1}(l, r, h, input))
    (P:537-539): pad the outer dimension(s) first, then the inner ones.  A
    per-dimension h is allowed (reading A10)."""
    P = np.asarray(x, dtype=np.float64)
    for d in range(P.ndim):
        P = pad1(P, d, pad_lo[d], pad_hi[d], kind[d], value, decay)
    return P


# ---------------------------------------------------------------------------
# slide and slide_n
# ---------------------------------------------------------------------------
def slide_count(n: int, size: int, step: int) -> int:
    """Number of windows of slide(size, step) over n elements:
    (n - size + step) / step, floor for a partial last window
    (reading A6).  0 when there is no full window."""
    if n < size:
        return 0
    return (n - size) // step + 1


def slide_tap(P: np.ndarray, k: Sequence[int], size: Sequence[int],
              step: Sequence[int]) -> np.ndarray:
    """Element k of every window: array over outputs o of P[o*step + k]."""
    sl = []
    for d in range(P.ndim):
        cnt = slide_count(P.shape[d], size[d], step[d])
        sl.append(slice(k[d], k[d] + step[d] * (cnt - 1) + 1, step[d]))
    return P[tuple(sl)]


def slide_n(P: np.ndarray, size: Sequence[int], step: Sequence[int]) -> np.ndarray:
    """Materialised neighbourhood array (small inputs only): shape
    ``out_extents + size`` with ``W[o..., k...] = P[o*step + k]`` — the
    n-dimensional neighbourhood after ``reorderingDimensions``."""
    outs = tuple(slide_count(P.shape[d], size[d], step[d]) for d in range(P.ndim))
    W = np.empty(outs + tuple(size), dtype=P.dtype)
    for k in np.ndindex(*size):
        W[(Ellipsis,) + k] = slide_tap(P, k, size, step)
    return W


# ---------------------------------------------------------------------------
# map: neighbourhood functions f.  ``W(k)`` returns element k of
# the window for all outputs (array) or for one output (scalar).
# ---------------------------------------------------------------------------
def f_weighted(W: Callable, weights: np.ndarray) -> Tuple:
    """Y = sum_k w_k * W[k] (Listing 2's reduce(add) over the neighbourhood,
    P:483, generalised with weights; cross-correlation, reading A7).
    Returns (Y, A) with A = sum_k |w_k * W[k]| (error scale, reading A22)."""
    w = np.asarray(weights, dtype=np.float64)
    Y = 0.0
    A = 0.0
    for k in np.ndindex(*w.shape):
        if w[k] == 0.0:
            continue
        t = w[k] * W(k)
        Y = Y + t
        A = A + np.abs(t)
    return Y, A


def _star(r: int, nd: int, d: int, off: int) -> Tuple[int, ...]:
    k = [r] * nd
    k[d] += off
    return tuple(k)


def f_hotspot3d(W: Callable, Pc, prm: Sequence[float]) -> Tuple:
    """Rodinia v3.1 hotspot3D update (reading A16, external; pinned by
    an independent scalar loop in tests/test_oracle_map.py):
    T' = cc*C + cn*N + cs*S + ce*E + cw*W + ct*T + cb*B + sdc*P + ct*amb,
    N=y-1, S=y+1, W=x-1, E=x+1, B=z-1, T=z+1 (clamped through the pad)."""
    cc, cn, cs, ce, cw, ct, cb, sdc, amb = (np.float64(v) for v in prm)
    C = W((1, 1, 1))
    terms = (cc * C, cn * W((1, 0, 1)), cs * W((1, 2, 1)), ce * W((1, 1, 2)),
             cw * W((1, 1, 0)), ct * W((2, 1, 1)), cb * W((0, 1, 1)),
             sdc * Pc, ct * amb)
    Y = 0.0
    A = 0.0
    for t in terms:
        Y = Y + t
        A = A + np.abs(t)
    return Y, A


def f_srad1(W: Callable, prm: Sequence[float]) -> Tuple:
    """Rodinia v3.1 SRAD first kernel, I -> c (reading A18, external; pinned by
    hand-derived closed forms: spike, face neighbour, ramp):
    dX = I_X - I_c;  G2 = sum dX^2 / I_c^2;  L = sum dX / I_c;
    num = 0.5*G2 - L^2/16;  den = 1 + 0.25*L;  q = num/den^2;
    d = (q - q0)/(q0*(1+q0));  c = clamp(1/(1+d), 0, 1)."""
    q0 = np.float64(prm[0])
    Ic = W((1, 1))
    dN = W((0, 1)) - Ic
    dS = W((2, 1)) - Ic
    dW = W((1, 0)) - Ic
    dE = W((1, 2)) - Ic
    G2 = (dN * dN + dS * dS + dW * dW + dE * dE) / (Ic * Ic)
    L = (dN + dS + dW + dE) / Ic
    num = 0.5 * G2 - (1.0 / 16.0) * (L * L)
    den = 1.0 + 0.25 * L
    q = num / (den * den)
    d = (q - q0) / (q0 * (1.0 + q0))
    c = 1.0 / (1.0 + d)
    c = np.clip(c, 0.0, 1.0)
    return c, np.abs(c)


def f_srad2(Wc: Callable, WI: Callable, prm: Sequence[float]) -> Tuple:
    """Rodinia v3.1 SRAD second kernel, (c, I) -> I' (reading A18; PARITY
    UNPINNED): D = c_c*dN + c_S*dS + c_c*dW + c_E*dE; I' = I_c + 0.25*lambda*D."""
    lam = np.float64(prm[0])
    Ic = WI((1, 1))
    dN = WI((0, 1)) - Ic
    dS = WI((2, 1)) - Ic
    dW = WI((1, 0)) - Ic
    dE = WI((1, 2)) - Ic
    cC = Wc((1, 1))
    cS = Wc((2, 1))
    cE = Wc((1, 2))
    terms = (cC * dN, cS * dS, cC * dW, cE * dE)
    D = terms[0] + terms[1] + terms[2] + terms[3]
    Y = Ic + 0.25 * lam * D
    A = np.abs(Ic) + 0.25 * lam * (np.abs(terms[0]) + np.abs(terms[1]) +
                                   np.abs(terms[2]) + np.abs(terms[3]))
    return Y, A


def srad_q0sqr(I: np.ndarray) -> float:
    """q0^2 = var(I) / mean(I)^2 over the whole image, fp64 (reading A18/A27)."""
    x = np.asarray(I, np.float64)
    m = x.mean()
    return float(x.var() / (m * m))


def srad_iteration(spec, I: np.ndarray):
    """One full SRAD iteration (reading A27, NEXT-2): q0^2 from the current
    image, c = SRAD1(I; q0^2), I' = SRAD2(c, I; lambda).  The diffusion
    coefficient c is a grid like any other: SRAD2 reads it through the same
    pad/slide.  Returns (I', A)."""
    q0 = srad_q0sqr(I)
    c, _ = apply(_with(spec, SRAD1, (q0,)), [I])
    return apply(_with(spec, SRAD2, (spec.params[0],)), [c, I])


def _with(spec, op, params):
    import copy
    s = copy.copy(spec)
    s.op = op
    s.params = tuple(params)
    return s


def f_hotspot2d(WT: Callable, WP: Callable, prm: Sequence[float]) -> Tuple:
    """Rodinia v3.1 hotspot (2D) update (reading A26, external; pinned by
    an independent scalar loop):
    T' = T + sdc*(P + (S + N - 2T)/Ry + (E + W - 2T)/Rx + (amb - T)/Rz),
    with params (sdc, 1/Rx, 1/Ry, 1/Rz, amb); N=y-1, S=y+1, W=x-1, E=x+1."""
    sdc, rx1, ry1, rz1, amb = (np.float64(v) for v in prm)
    T = WT((1, 1))
    terms = (WP((1, 1)), (WT((2, 1)) + WT((0, 1)) - 2.0 * T) * ry1,
             (WT((1, 2)) + WT((1, 0)) - 2.0 * T) * rx1, (amb - T) * rz1)
    acc = terms[0] + terms[1] + terms[2] + terms[3]
    Y = T + sdc * acc
    aT = np.abs(T)
    A = aT + np.abs(sdc) * (np.abs(terms[0]) + (np.abs(WT((2, 1))) + np.abs(WT((0, 1))) + 2.0 * aT) * abs(ry1) +
                            (np.abs(WT((1, 2))) + np.abs(WT((1, 0))) + 2.0 * aT) * abs(rx1) +
                            (abs(amb) + aT) * abs(rz1))
    return Y, A


def f_gradient(W: Callable, prm: Sequence[float]) -> Tuple:
    """Rawat et al. [36] 2D gradient (reading A25, external; pinned by
    an independent scalar loop):
    out = I + 1/sqrt(eps + (I-N)^2 + (I-S)^2 + (I-W)^2 + (I-E)^2)."""
    eps = np.float64(prm[0])
    Ic = W((1, 1))
    s = eps + (Ic - W((0, 1))) ** 2 + (Ic - W((2, 1))) ** 2 + (Ic - W((1, 0))) ** 2 + (Ic - W((1, 2))) ** 2
    Y = Ic + 1.0 / np.sqrt(s)
    return Y, np.abs(Ic) + np.abs(1.0 / np.sqrt(s))


def acoustic_neighbours(o: Sequence, extents: Sequence[int], r: int):
    """computeNumNeighbors (Listing 3 line 14; reading A19):
    K = number of the star neighbour offsets (+-1..+-r on each axis) whose
    target lies inside the domain.  Works on arrays of indices (broadcast)."""
    K = 0
    for d in range(len(extents)):
        for off in range(1, r + 1):
            for sgn in (-1, 1):
                j = np.asarray(o[d]) + sgn * off
                K = K + ((j >= 0) & (j < extents[d])).astype(np.int64)
    return K


def f_acoustic(W: Callable, prev_c, K, r: int, prm: Sequence[float]) -> Tuple:
    """Listing 3 with the physics reading A19 (slid grid = u^n,
    point-wise grid = u^{n-1}, output = u^{n+1}; the constants are proposed;
    roles pinned by the leapfrog identity and per-grid locality):
    u' = cf(K, l1) * ((2 - l2*K) * u_c + l2 * sum_nbr u - cf(K, l2loss) * prev),
    getCF(K, x, 1.0) = (K < K_max) ? x : 1.0."""
    l2, loss1, loss2 = (np.float64(v) for v in prm)
    kmax = 6 * r
    c = (r, r, r)
    s = 0.0
    sabs = 0.0
    for k in np.ndindex(*(2 * r + 1,) * 3):
        # star neighbours only, in row-major tap order (Listing 3 lines 5-6)
        dev = [k[d] - r for d in range(3)]
        if sum(1 for v in dev if v != 0) != 1:
            continue
        v = W(k)
        s = s + v
        sabs = sabs + np.abs(v)
    uc = W(c)
    cf1 = np.where(K < kmax, loss1, 1.0)
    cf2 = np.where(K < kmax, loss2, 1.0)
    t0 = (2.0 - l2 * K) * uc
    t1 = l2 * s
    t2 = cf2 * prev_c
    Y = cf1 * (t0 + t1 - t2)
    A = np.abs(cf1) * (np.abs(t0) + l2 * sabs + np.abs(t2))
    return Y, A


# ---------------------------------------------------------------------------
# apply / iterate
# ---------------------------------------------------------------------------
def _check_op_shape(spec):
    if spec.op in (HOTSPOT3D, ACOUSTIC):
        assert spec.ndim == 3
    if spec.op in (SRAD1, SRAD2, HOTSPOT2D, GRADIENT, SRAD):
        assert spec.ndim == 2
    if spec.op != WEIGHTED:
        assert all(s == 1 for s in spec.step)
        r = spec.size[0] // 2
        assert all(s == 2 * r + 1 for s in spec.size)
        assert all(l == r and h == r for l, h in zip(spec.pad_lo, spec.pad_hi))


def apply(spec, inputs: Sequence[np.ndarray]):
    """One application of the stencil: returns (Y, A) as fp64 arrays of the
    output extents; A is the absolute-term error scale (reading A22)."""
    _check_op_shape(spec)
    pad = lambda x: pad_n(x, spec.pad_lo, spec.pad_hi, spec.kind, spec.pad_value, getattr(spec, "pad_decay", 1.0))
    tapper = lambda P: (lambda k: slide_tap(P, k, spec.size, spec.step))
    outs = spec.out_extents()
    if spec.op == WEIGHTED:
        Y, A = f_weighted(tapper(pad(inputs[0])), spec.weights)
    elif spec.op == HOTSPOT3D:
        Y, A = f_hotspot3d(tapper(pad(inputs[0])), inputs[1].astype(np.float64), spec.params)
    elif spec.op == SRAD1:
        Y, A = f_srad1(tapper(pad(inputs[0])), spec.params)
    elif spec.op == SRAD2:
        Y, A = f_srad2(tapper(pad(inputs[0])), tapper(pad(inputs[1])), spec.params)
    elif spec.op == SRAD:
        Y, A = srad_iteration(spec, inputs[0])
    elif spec.op == HOTSPOT2D:
        Y, A = f_hotspot2d(tapper(pad(inputs[0])), tapper(pad(inputs[1])), spec.params)
    elif spec.op == GRADIENT:
        Y, A = f_gradient(tapper(pad(inputs[0])), spec.params)
    elif spec.op == ACOUSTIC:
        r = spec.size[0] // 2
        o = np.meshgrid(*[np.arange(n) for n in outs], indexing="ij", sparse=True)
        K = acoustic_neighbours(o, spec.extents, r)
        prev, cur = inputs
        Y, A = f_acoustic(tapper(pad(cur)), prev.astype(np.float64), K, r, spec.params)
    else:
        raise ValueError(spec.op)
    Y = np.broadcast_to(np.asarray(Y, np.float64), outs).copy()
    A = np.broadcast_to(np.asarray(A, np.float64), outs).copy()
    return Y, A


def apply_point(spec, inputs: Sequence[np.ndarray], o: Sequence[int]):
    """One output point computed directly from the index functions, without
    materialising the padded grid (for sampled parity at full sizes).  The
    same definition as ``apply``: padded index p = o*step + k, input index
    p - l remapped by h, or the constant."""
    _check_op_shape(spec)

    def fetch(x, k):
        # pad_n pads the outer dimension first, so the cell seen
        # through an inner pad is resolved first: walk the dimensions innermost
        # first — a CONSTANT dimension outside ends the walk with the value,
        # DAMPEN contributes decay^distance (reading A29)
        idx = [0] * spec.ndim
        factor = np.float64(1.0)
        for d in reversed(range(spec.ndim)):
            i = int(o[d]) * spec.step[d] + k[d] - spec.pad_lo[d]
            n = spec.extents[d]
            if i < 0 or i >= n:
                if spec.kind[d] == CONSTANT:
                    return np.float64(spec.pad_value) * factor
                if spec.kind[d] == DAMPEN:
                    factor *= np.float64(getattr(spec, "pad_decay", 1.0)) ** int(dampen_distance(i, n))
                    i = int(h_clamp(i, n))
                else:
                    i = int(H[spec.kind[d]](i, n))
            idx[d] = i
        return np.float64(x[tuple(idx)]) * factor

    tap = lambda x: (lambda k: fetch(x, k))
    if spec.op == WEIGHTED:
        return f_weighted(tap(inputs[0]), spec.weights)
    if spec.op == HOTSPOT3D:
        return f_hotspot3d(tap(inputs[0]), np.float64(inputs[1][tuple(o)]), spec.params)
    if spec.op == SRAD1:
        return f_srad1(tap(inputs[0]), spec.params)
    if spec.op == SRAD2:
        return f_srad2(tap(inputs[0]), tap(inputs[1]), spec.params)
    if spec.op == HOTSPOT2D:
        return f_hotspot2d(tap(inputs[0]), tap(inputs[1]), spec.params)
    if spec.op == GRADIENT:
        return f_gradient(tap(inputs[0]), spec.params)
    if spec.op == ACOUSTIC:
        r = spec.size[0] // 2
        K = acoustic_neighbours(o, spec.extents, r)
        return f_acoustic(tap(inputs[1]), np.float64(inputs[0][tuple(o)]), K, r, spec.params)
    raise ValueError(spec.op)


def pad_planes(x: np.ndarray, p0: int, p1: int, l: int, kind: int, value: float = 0.0,
               decay: float = 1.0) -> np.ndarray:
    """Padded planes p0 .. p1-1 of ``pad1(x, 0, l, *, kind)`` along axis 0,
    without materialising the rest: padded plane p reads x[h(p - l, n)], the
    constant, or the nearest plane times decay^d (the same definitions as
    pad1, readings A1-A5, A29), in fp64."""
    n = x.shape[0]
    planes = []
    for p in range(p0, p1):
        i = p - l
        if 0 <= i < n:
            planes.append(np.asarray(x[i], np.float64))
        elif kind == CONSTANT:
            planes.append(np.full(x.shape[1:], np.float64(value)))
        elif kind == DAMPEN:
            planes.append(np.asarray(x[int(h_clamp(i, n))], np.float64) *
                          np.float64(decay) ** int(dampen_distance(i, n)))
        else:
            planes.append(np.asarray(x[int(H[kind](i, n))], np.float64))
    return np.stack(planes, 0)


def apply_planes(spec, inputs: Sequence[np.ndarray], z0: int, z1: int):
    """Output planes [z0, z1) of dimension 0 of ``apply`` (for full-grid checks
    of grids too large to pad at once).  The same definition restricted to a
    block of outputs: output plane o reads padded planes o*step_0 + k
    (slide), so the block needs padded planes
    [z0*step_0, (z1-1)*step_0 + size_0); those are built by ``pad_planes``
    (dimension 0 first, as pad_n), the inner dimensions are padded
    by pad_n, and the map is the same f.  Point-wise grids are taken at the
    output planes; Acoustic's K uses the global extents and plane index."""
    _check_op_shape(spec)
    if spec.op == SRAD:
        raise ValueError("the SRAD iteration's q0 is a whole-image statistic: use apply")
    decay = getattr(spec, "pad_decay", 1.0)
    p0 = z0 * spec.step[0]
    p1 = (z1 - 1) * spec.step[0] + spec.size[0]
    inner_lo = (0,) + tuple(spec.pad_lo[1:])
    inner_hi = (0,) + tuple(spec.pad_hi[1:])

    def pad(x):
        P0 = pad_planes(x, p0, p1, spec.pad_lo[0], spec.kind[0], spec.pad_value, decay)
        return pad_n(P0, inner_lo, inner_hi, spec.kind, spec.pad_value, decay)

    sub_step = (spec.step[0],) + tuple(spec.step[1:])
    tapper = lambda P: (lambda k: slide_tap(P, k, spec.size, sub_step))
    outs = (z1 - z0,) + tuple(spec.out_extents()[1:])
    if spec.op == WEIGHTED:
        Y, A = f_weighted(tapper(pad(inputs[0])), spec.weights)
    elif spec.op == HOTSPOT3D:
        Y, A = f_hotspot3d(tapper(pad(inputs[0])), np.asarray(inputs[1][z0:z1], np.float64), spec.params)
    elif spec.op == SRAD1:
        Y, A = f_srad1(tapper(pad(inputs[0])), spec.params)
    elif spec.op == SRAD2:
        Y, A = f_srad2(tapper(pad(inputs[0])), tapper(pad(inputs[1])), spec.params)
    elif spec.op == HOTSPOT2D:
        Y, A = f_hotspot2d(tapper(pad(inputs[0])), tapper(pad(inputs[1])), spec.params)
    elif spec.op == GRADIENT:
        Y, A = f_gradient(tapper(pad(inputs[0])), spec.params)
    elif spec.op == ACOUSTIC:
        r = spec.size[0] // 2
        full = spec.out_extents()
        o = np.meshgrid(np.arange(z0, z1), *[np.arange(n) for n in full[1:]], indexing="ij", sparse=True)
        K = acoustic_neighbours(o, spec.extents, r)
        prev, cur = inputs
        Y, A = f_acoustic(tapper(pad(cur)), np.asarray(prev[z0:z1], np.float64), K, r, spec.params)
    else:
        raise ValueError(spec.op)
    Y = np.broadcast_to(np.asarray(Y, np.float64), outs).copy()
    A = np.broadcast_to(np.asarray(A, np.float64), outs).copy()
    return Y, A


def iterate(spec, state: Sequence[np.ndarray], aux: Sequence[np.ndarray], n_steps: int,
            round_fp32: bool = False):
    """iterate(in, f, m) with the state rotation of reading
    A21: WEIGHTED X <- S(X); HOTSPOT3D T <- S(T, P), P fixed; ACOUSTIC
    (prev, cur) <- (cur, S(prev, cur)).  Returns the final state in fp64
    (the newest grid last).  ``round_fp32`` rounds each step's output to fp32
    before feeding it back (not used by the parity tests: the oracle keeps
    fp64 state)."""
    cvt = (lambda a: a.astype(np.float32).astype(np.float64)) if round_fp32 else (lambda a: a)
    if spec.op in (WEIGHTED, HOTSPOT3D, HOTSPOT2D, GRADIENT, SRAD):
        X = np.asarray(state[0], np.float64)
        for _ in range(n_steps):
            X, _A = apply(spec, [X] + list(aux))
            X = cvt(X)
        return [X]
    if spec.op == ACOUSTIC:
        prev = np.asarray(state[0], np.float64)
        cur = np.asarray(state[1], np.float64)
        for _ in range(n_steps):
            nxt, _A = apply(spec, [prev, cur])
            prev, cur = cur, cvt(nxt)
        return [prev, cur]
    raise ValueError("iterate is defined for WEIGHTED, HOTSPOT3D, ACOUSTIC")


def max_rel_err(g: np.ndarray, Y: np.ndarray, A: np.ndarray) -> float:
    """err_p = |g_p - o_p| / max(|o_p|, A_p) (reading A22)."""
    g = np.asarray(g, np.float64)
    den = np.maximum(np.abs(Y), A)
    den = np.where(den == 0.0, 1.0, den)
    return float(np.max(np.abs(g - Y) / den)) if g.size else 0.0
