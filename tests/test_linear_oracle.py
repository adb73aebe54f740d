"""Pins of the general linear-stencil oracle (oracle.c `oracle_linear`: any access set, any
radius, A'[p] = sum_k c_k A[p + o_k] left to right over [R, N-1-R]) -- against what mathematics
and the already-pinned class oracles fix, not against a retyped formula:
  * with coefficient 1 and the classes' own access orders it IS the box / Jacobi sums of the
    pinned class oracles (multiplication by 1 is exact, the additions happen in the same order),
    bit for bit on arbitrary inputs;
  * with dyadic coefficients and small integer inputs every operation is exact, so any summation
    order gives the same value: iterated scipy.ndimage.correlate (a library routine);
  * coefficients summing to 1 keep a constant field 1.0 exactly (Dirichlet boundary included)."""
import itertools

import numpy as np
import pytest

import oracle
import stencil_inputs

scipy_ndimage = pytest.importorskip("scipy.ndimage")


def test_unit_box2d9_equals_class_oracle_bitwise():
    offs = [(a, b) for a in (-1, 0, 1) for b in (-1, 0, 1)]  # row-major: the box2d9 order
    g = stencil_inputs.uniform((23, 31), seed=4)
    got = oracle.linear(g, offs, [1.0] * 9, 6)
    exp = oracle.run("box2d9", g, 6, coef=(1.0,))
    assert np.array_equal(got, exp)


def test_unit_box3d27_equals_class_oracle_bitwise():
    offs = list(itertools.product((-1, 0, 1), repeat=3))  # lexicographic: the box3d27 order
    g = stencil_inputs.uniform((9, 10, 12), seed=5, dtype=np.float64)
    got = oracle.linear(g, offs, [1.0] * 27, 4)
    exp = oracle.run("box3d27", g, 4, coef=(1.0,))
    assert np.array_equal(got, exp)


def test_unit_jacobi_order_equals_class_oracle_bitwise():
    """Fig. 1's operand order c, s, n, e, w with k = 1."""
    offs = [(0, 0), (1, 0), (-1, 0), (0, 1), (0, -1)]
    g = stencil_inputs.uniform((17, 29), seed=6)
    got = oracle.linear(g, offs, [1.0] * 5, 7)
    exp = oracle.run("jacobi2d5", g, 7, coef=(1.0,))
    assert np.array_equal(got, exp)


def _correlate_steps(g, offs, coefs, steps):
    """Iterated correlation over the interior [R, N-1-R], boundary cells fixed."""
    R = max(abs(o) for off in offs for o in off)
    size = 2 * R + 1
    w = np.zeros((size,) * g.ndim)
    for off, c in zip(offs, coefs):
        w[tuple(o + R for o in off)] += c
    a = g.astype(np.float64).copy()
    inner = tuple(slice(R, n - R) for n in g.shape)
    for _ in range(steps):
        nxt = a.copy()
        nxt[inner] = scipy_ndimage.correlate(a, w, mode="constant", cval=0.0)[inner]
        a = nxt
    return a


STAR2D_R2 = [(0, 0), (-1, 0), (1, 0), (0, -1), (0, 1), (-2, 0), (2, 0), (0, -2), (0, 2)]
UPWIND2D = [(0, 0), (0, -1), (0, -2), (-1, 0)]
STAR3D_R2 = [(0, 0, 0), (-2, 0, 0), (2, 0, 0), (0, -1, 0), (0, 1, 0), (0, 0, -2), (0, 0, 2), (1, 1, 1)]


@pytest.mark.parametrize("offs,coefs,shape,steps", [
    (STAR2D_R2, [0.5, 0.125, 0.0625, 0.125, 0.0625, 0.03125, 0.03125, 0.0625, 0.0625], (14, 15), 3),
    (UPWIND2D, [0.25, 0.5, 0.125, 0.125], (12, 13), 4),
    (STAR3D_R2, [0.5, 0.0625, 0.0625, 0.125, 0.0625, 0.03125, 0.0625, 0.125], (11, 9, 10), 3),
])
def test_exact_dyadic_equals_scipy_correlate(offs, coefs, shape, steps):
    rng = np.random.default_rng(3)
    g = rng.integers(-3, 4, size=shape).astype(np.float64)
    got = oracle.linear(g, offs, coefs, steps)
    exp = _correlate_steps(g, offs, coefs, steps)
    assert np.array_equal(got, exp)


@pytest.mark.parametrize("dtype", [np.float32, np.float64])
def test_constant_field_fixpoint(dtype):
    g = np.ones((16, 18), dtype=dtype)
    coefs = [0.5, 0.125, 0.0625, 0.125, 0.0625, 0.03125, 0.03125, 0.03125, 0.03125]
    assert sum(coefs) == 1.0
    assert np.array_equal(oracle.linear(g, STAR2D_R2, coefs, 9), g)


def test_radius_sets_the_dirichlet_margin():
    """Cells within R = max |offset| of an edge are never written (R = 2 here)."""
    g = stencil_inputs.uniform((12, 13), seed=8, dtype=np.float64)
    got = oracle.linear(g, STAR2D_R2, [1.0 / 9] * 9, 3)
    for sl in [(slice(0, 2), slice(None)), (slice(-2, None), slice(None)), (slice(None), slice(0, 2)),
               (slice(None), slice(-2, None))]:
        assert np.array_equal(got[sl], g[sl])
    assert not np.array_equal(got[2:-2, 2:-2], g[2:-2, 2:-2])
