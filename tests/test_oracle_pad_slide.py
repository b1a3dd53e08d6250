"""Pins for the oracle's pad / pad_n / slide / slide_n (CPU, no GPU).

Each test checks the oracle against something other than itself: numpy.pad
modes, numpy's sliding_window_view, the paper's printed examples
(tests/golden/, Fig. 3),
and scalar brute force written from the paper's clamp definition.
"""
import itertools
import json
import os

import numpy as np
import pytest
from numpy.lib.stride_tricks import sliding_window_view

import oracle
from oracle.stencil_oracle import (CLAMP, CONSTANT, MIRROR, REFLECT, WRAP, pad1, pad_n,
                                   slide_count, slide_n, slide_tap)

GOLD = os.path.join(os.path.dirname(__file__), "golden")
NP_MODE = {CLAMP: "edge", MIRROR: "symmetric", WRAP: "wrap", REFLECT: "reflect"}


def gold(name):
    with open(os.path.join(GOLD, name)) as f:
        return json.load(f)


def symbolic(arr):
    """Map a nested list of symbols to (float array, inverse table)."""
    a = np.array(arr)
    syms = sorted(set(a.ravel().tolist()))
    table = {s: float(i + 1) for i, s in enumerate(syms)}
    return np.vectorize(table.get)(a).astype(np.float64), {v: k for k, v in table.items()}


# ---------------------------------------------------------------- pad ------
@pytest.mark.parametrize("kind", [CLAMP, MIRROR, WRAP, REFLECT])
def test_pad1_matches_numpy_modes(kind):
    rng = np.random.default_rng(0)
    for n in range(1, 9):
        x = rng.random(n)
        for l, r in itertools.product(range(5), range(5)):
            if kind == REFLECT and n == 1 and (l or r):
                continue  # numpy 'reflect' on one element: compared below
            got = pad1(x, 0, l, r, kind)
            exp = np.pad(x, (l, r), mode=NP_MODE[kind])
            np.testing.assert_array_equal(got, exp, err_msg=f"n={n} l={l} r={r} kind={kind}")


def test_pad1_reflect_single_element_is_constant_extension():
    x = np.array([3.5])
    np.testing.assert_array_equal(pad1(x, 0, 3, 2, REFLECT), np.full(6, 3.5))


def test_pad1_constant_matches_numpy():
    rng = np.random.default_rng(1)
    for n in range(1, 9):
        x = rng.random(n)
        for l, r in itertools.product(range(5), range(5)):
            got = pad1(x, 0, l, r, CONSTANT, 0.625)
            exp = np.pad(x, (l, r), mode="constant", constant_values=0.625)
            np.testing.assert_array_equal(got, exp)


def test_clamp_brute_force_from_paper_definition():
    """clamp(i, n) = (i < 0) ? 0 : ((i >= n) ? n-1 : i), as a scalar
    if-chain, against the oracle's vectorised pad."""
    def clamp(i, n):
        if i < 0:
            return 0
        if i >= n:
            return n - 1
        return i
    rng = np.random.default_rng(2)
    for n in range(1, 8):
        x = rng.random(n)
        for l, r in itertools.product(range(6), range(6)):
            exp = [x[clamp(j - l, n)] for j in range(l + n + r)]
            np.testing.assert_array_equal(pad1(x, 0, l, r, CLAMP), exp)


def test_pad_2_3_clamp_paper_text():
    g = gold("pad_2_3_clamp_P452.json")
    got = pad1(np.array(g["input"], np.float64), 0, 2, 3, CLAMP)
    np.testing.assert_array_equal(got, g["expected"])
    assert got.shape[0] == 2 + len(g["input"]) + 3          # type [T]_{l+n+r}


def test_pad2_clamp_paper_example():
    g = gold("pad2_clamp_P546.json")
    x, inv = symbolic(g["input"])
    outer = pad1(x, 0, 1, 1, CLAMP)
    assert np.vectorize(inv.get)(outer).tolist() == g["intermediate_outer_pad"]
    got = pad_n(x, (1, 1), (1, 1), (CLAMP, CLAMP))
    assert np.vectorize(inv.get)(got).tolist() == g["expected"]


@pytest.mark.parametrize("kind", [CLAMP, MIRROR, WRAP, CONSTANT, REFLECT])
def test_pad_identity_in_range(kind):
    """h must be the identity in range: pad(X)[l:l+n] == X."""
    rng = np.random.default_rng(3)
    x = rng.random((5, 7, 6))
    P = pad_n(x, (2, 1, 3), (1, 4, 2), (kind,) * 3, 0.3)
    np.testing.assert_array_equal(P[2:7, 1:8, 3:9], x)
    assert P.shape == (5 + 3, 7 + 5, 6 + 5)


def _pad_inner_first(x, lo, hi, kinds, value):
    P = np.asarray(x, np.float64)
    for d in reversed(range(P.ndim)):
        P = pad1(P, d, lo[d], hi[d], kinds[d], value)
    return P


def test_pad_n_order_independence_mixed_kinds():
    """Reading A9: outer-first == inner-first for every pair of
    kinds, including CONSTANT corners (brute force)."""
    rng = np.random.default_rng(4)
    kinds = [CLAMP, MIRROR, WRAP, CONSTANT, REFLECT]
    for shape in [(3, 4), (1, 5), (4, 2)]:
        x = rng.random(shape)
        for k0, k1 in itertools.product(kinds, kinds):
            for lo, hi in [((1, 2), (2, 1)), ((3, 0), (0, 3)), ((4, 4), (5, 2))]:
                a = pad_n(x, lo, hi, (k0, k1), 0.7)
                b = _pad_inner_first(x, lo, hi, (k0, k1), 0.7)
                np.testing.assert_array_equal(a, b)


def test_pad_n_matches_numpy_3d_per_dim():
    rng = np.random.default_rng(5)
    x = rng.random((3, 4, 5))
    for kinds in itertools.product([CLAMP, MIRROR, WRAP, REFLECT], repeat=3):
        lo, hi = (2, 1, 3), (1, 3, 2)
        exp = x
        for d in range(3):
            pw = [(0, 0)] * 3
            pw[d] = (lo[d], hi[d])
            exp = np.pad(exp, pw, mode=NP_MODE[kinds[d]])
        np.testing.assert_array_equal(pad_n(x, lo, hi, kinds), exp)


# -------------------------------------------------------------- slide ------
def test_slide_count_matches_sliding_window_view():
    """(n - size + step)/step windows, floor rule (A6)."""
    for n in range(1, 13):
        for size in range(1, 6):
            for step in range(1, 4):
                if size > n:
                    assert slide_count(n, size, step) == 0
                    continue
                exp = sliding_window_view(np.arange(n), size)[::step].shape[0]
                assert slide_count(n, size, step) == exp
                if (n - size) % step == 0:
                    assert slide_count(n, size, step) == (n - size + step) // step


def test_slide1_windows_match_sliding_window_view():
    x = np.arange(11, dtype=np.float64)
    for size in range(1, 6):
        for step in range(1, 4):
            W = slide_n(x, (size,), (step,))
            np.testing.assert_array_equal(W, sliding_window_view(x, size)[::step])


def test_slide2_paper_example():
    g = gold("slide2_P575.json")
    x, inv = symbolic(g["input"])
    W = slide_n(x, (2, 2), (1, 1))
    assert np.vectorize(inv.get)(W).tolist() == g["expected"]


def test_slide_n_matches_sliding_window_view_nd():
    rng = np.random.default_rng(6)
    x = rng.random((7, 8, 9))
    for size, step in [((3, 3, 3), (1, 1, 1)), ((2, 3, 4), (2, 1, 3)), ((5, 1, 2), (1, 2, 2))]:
        W = slide_n(x, size, step)
        exp = sliding_window_view(x, size)[::step[0], ::step[1], ::step[2]]
        np.testing.assert_array_equal(W, exp)


def test_fig3_pipeline_windows():
    g = gold("fig3_P427.json")
    P = pad_n(np.array(g["input"], np.float64), (1,), (1,), (CLAMP,))
    W = slide_n(P, (3,), (1,))
    assert W.shape[0] == g["n_windows"]
    for k, v in g["legible_windows"].items():
        np.testing.assert_array_equal(W[int(k)], v)


def test_overlapped_tiling_rule_listing4():
    """Listing 4 / tiling rule: slide(5,3) tiles, then
    slide(3,1) inside each tile, joined, equals slide(3,1) directly
    (size - step = u - v).  Pins that the oracle's slide composes as stated."""
    x = np.arange(14, dtype=np.float64)   # padded length 14: (14 - 5) / 3 + 1 = 4 tiles
    direct = slide_n(x, (3,), (1,))
    tiles = slide_n(x, (5,), (3,))
    tiled = np.concatenate([slide_n(t, (3,), (1,)) for t in tiles])
    np.testing.assert_array_equal(tiled, direct)


def test_slide_tap_is_window_element():
    rng = np.random.default_rng(7)
    P = rng.random((6, 9))
    W = slide_n(P, (3, 2), (2, 3))
    for k in np.ndindex(3, 2):
        np.testing.assert_array_equal(slide_tap(P, k, (3, 2), (2, 3)), W[..., k[0], k[1]])


# ------------------------------------- DAMPEN value pad (reading A29) ------
def test_dampen_special_cases_are_edge_and_zero_padding():
    """decay 1 is numpy 'edge' (CLAMP), decay 0 is zero padding."""
    from oracle.stencil_oracle import DAMPEN
    rng = np.random.default_rng(41)
    for n in range(1, 7):
        x = rng.random(n)
        for l, r in itertools.product(range(4), range(4)):
            np.testing.assert_array_equal(pad1(x, 0, l, r, DAMPEN, decay=1.0), np.pad(x, (l, r), mode="edge"))
            np.testing.assert_array_equal(pad1(x, 0, l, r, DAMPEN, decay=0.0), np.pad(x, (l, r)))


def test_dampen_brute_force_2d_and_mixed_with_constant():
    """Per cell: the nearest element times decay^(cells outside), summed over
    the DAMPEN dimensions; a CONSTANT dimension outside gives c times decay^
    (cells outside in the dimensions padded after it, pad_n's order P:537-539)."""
    from oracle.stencil_oracle import DAMPEN
    x = np.arange(12, dtype=np.float64).reshape(3, 4) + 1.0
    g, c = 0.5, 7.0
    dist = lambda i, n: -i if i < 0 else (i - n + 1 if i >= n else 0)
    cl = lambda i, n: min(max(i, 0), n - 1)
    P = pad_n(x, (2, 1), (1, 3), (DAMPEN, DAMPEN), decay=g)
    for a, b in itertools.product(range(6), range(8)):
        i, j = a - 2, b - 1
        assert P[a, b] == x[cl(i, 3), cl(j, 4)] * g ** (dist(i, 3) + dist(j, 4))
    Q = pad_n(x, (2, 1), (1, 3), (CONSTANT, DAMPEN), value=c, decay=g)
    for a, b in itertools.product(range(6), range(8)):
        i, j = a - 2, b - 1
        base = c if not 0 <= i < 3 else x[i, cl(j, 4)]
        assert Q[a, b] == base * g ** dist(j, 4)
    R = pad_n(x, (2, 1), (1, 3), (DAMPEN, CONSTANT), value=c, decay=g)
    for a, b in itertools.product(range(6), range(8)):
        i, j = a - 2, b - 1
        assert R[a, b] == (c if not 0 <= j < 4 else x[cl(i, 3), j] * g ** dist(i, 3))


def test_dampen_apply_point_equals_apply():
    import stencil_inputs as si
    from oracle import stencil_oracle as orc
    rng = np.random.default_rng(42)
    for kinds in [(si.DAMPEN, si.DAMPEN, si.DAMPEN), (si.CONSTANT, si.DAMPEN, si.WRAP),
                  (si.DAMPEN, si.CONSTANT, si.DAMPEN), (si.MIRROR, si.DAMPEN, si.CONSTANT)]:
        x = rng.random((5, 6, 7))
        w = rng.standard_normal((3, 4, 3)).astype(np.float32)
        sp = si.StencilSpec((5, 6, 7), (3, 4, 3), (2, 1, 2), (2, 3, 1), (1, 2, 2), kinds, 0.375, si.WEIGHTED,
                            w, (), pad_decay=0.625)
        Y, A = orc.apply(sp, [x])
        for o in np.ndindex(*Y.shape):
            y, a = orc.apply_point(sp, [x], o)
            assert y == pytest.approx(Y[o], rel=1e-13, abs=1e-13)
