"""Pins of the CPU oracle (oracle/oracle.c) against what the paper and the mathematics fix,
so that a plausible mistake anywhere in it (dropped term, wrong sign or index, wrong
coefficient, wrong statement order, broken ping-pong) fails at least one test.

Each test names what it pins.  None of them compares the oracle with a re-typing of its
own formula."""
from fractions import Fraction

import numpy as np
import pytest
import scipy.ndimage
import scipy.sparse

import oracle
import stencil_inputs
from conftest import read_golden

LINEAR = ["jacobi2d5", "star2d5", "box2d9", "star3d7", "box3d27"]


def kernel_weights(kind, coef=None):
    """Correlation weights of a linear class as an explicit dense kernel (the stencil's
    offsets and coefficients, Table 3 / Fig. 1), for library cross-checks."""
    c = oracle.DEFAULT_COEF[kind] if coef is None else coef
    if kind == "jacobi2d5":
        w = np.zeros((3, 3)); w[1, 1] = w[0, 1] = w[2, 1] = w[1, 0] = w[1, 2] = c[0]
    elif kind == "star2d5":
        w = np.zeros((3, 3)); w[0, 1] = w[2, 1] = w[1, 0] = w[1, 2] = c[1]; w[1, 1] = c[0]
    elif kind == "box2d9":
        w = np.full((3, 3), c[0])
    elif kind == "star3d7":
        w = np.zeros((3, 3, 3))
        for o in [(0, 1, 1), (2, 1, 1), (1, 0, 1), (1, 2, 1), (1, 1, 0), (1, 1, 2)]:
            w[o] = c[1]
        w[1, 1, 1] = c[0]
    elif kind == "box3d27":
        w = np.full((3, 3, 3), c[0])
    return w


def interior(shape):
    return tuple(slice(1, n - 1) for n in shape)


# --- Fig. 1 / Fig. 2 golden ------------------------------------------------------------

def test_jacobi_fig1_fig2_golden_impulse():
    """Pins Fig. 1's stencil (5 points, 0.2 scale, loops 1..N-2) and Fig. 2's fp32
    constant 0f3E4CCCCD with hand-worked exact values (tests/golden/jacobi2d5_8x8_impulse.txt)."""
    rows = read_golden("jacobi2d5_8x8_impulse.txt")
    for dtype in (np.float32, np.float64):
        a = np.zeros((8, 8), dtype)
        a[3, 3] = 1
        for step in (1, 2):
            exp = np.zeros((8, 8))
            for s, i, j, num, den in rows:
                if int(s) == step:
                    exp[int(i), int(j)] = float(Fraction(int(num), int(den)))
            got = oracle.run("jacobi2d5", a, step).astype(np.float64)
            ulp = np.spacing(np.abs(exp).astype(dtype)).astype(np.float64)
            assert np.all(np.abs(got - exp) <= 2 * ulp + 0.0), (dtype, step)
    # step 1 in fp32: sum = 1 exactly, times 0.2f -> exactly the Fig. 2 constant bits
    a = np.zeros((8, 8), np.float32); a[3, 3] = 1
    r1 = oracle.run("jacobi2d5", a, 1).view(np.uint32)
    for i, j in [(3, 3), (2, 3), (4, 3), (3, 2), (3, 4)]:
        assert r1[i, j] == 0x3E4CCCCD


def test_jacobi_fig2_operation_order_fp32():
    """Fig. 2: four add.f32 in Fig. 1's operand order (c, i+1, i-1,
    j+1, j-1), then one mul.f32 by 0f3E4CCCCD.  Values chosen so that other
    associations round differently."""
    a = np.zeros((5, 5), np.float32)
    a[2, 2], a[3, 2], a[1, 2], a[2, 3], a[2, 1] = 1.0, 3e-8, 3e-8, 2.0**-24, 1e-8
    got = oracle.run("jacobi2d5", a, 1)[2, 2]
    f = np.float32
    s = f(f(f(f(f(1.0) + f(3e-8)) + f(3e-8)) + f(2.0**-24)) + f(1e-8))
    assert got.view(np.uint32) == f(np.float32(np.uint32(0x3E4CCCCD).view(np.float32)) * s).view(np.uint32)
    other = f(f(1.0) + f(f(f(3e-8) + f(3e-8)) + f(f(2.0**-24) + f(1e-8))))
    assert other != s  # the test input distinguishes association orders


def test_fdtd_golden_impulse_statement_order():
    """Pins the three FDTD statements, their coefficients, index directions and the
    ey -> ex -> hz order (tests/golden/fdtd2d_impulse.txt, hand-worked)."""
    rows = read_golden("fdtd2d_impulse.txt")
    for dtype in (np.float32, np.float64):
        z = np.zeros((8, 8), dtype)
        hz = z.copy(); hz[3, 3] = 1
        ex, ey, hz1 = oracle.fdtd(z, z, hz, 1)
        exp = {"ex": np.zeros((8, 8)), "ey": np.zeros((8, 8)), "hz": np.zeros((8, 8))}
        for f, i, j, num, den in rows:
            exp[f][int(i), int(j)] = float(Fraction(int(num), int(den)))
        tol = 4 * np.finfo(dtype).eps
        np.testing.assert_allclose(ex, exp["ex"], atol=tol)
        np.testing.assert_allclose(ey, exp["ey"], atol=tol)
        np.testing.assert_allclose(hz1, exp["hz"], atol=tol)


# --- invariants / closed forms ----------------------------------------------------------

@pytest.mark.parametrize("kind", LINEAR + ["gradient2d", "gradient3d"])
@pytest.mark.parametrize("dtype", [np.float32, np.float64])
def test_constant_field(kind, dtype):
    """A constant field 1.0 is a fixpoint of every linear class (coefficients sum to 1);
    for gradient every point strictly inside the t-cone of the boundary grows by exactly
    fl(1/fl(sqrt(eps))) per step."""
    shape = (12, 12) if oracle.DIMS[kind] == 2 else (12, 12, 12)
    a = np.ones(shape, dtype)
    steps = 4
    out = oracle.run(kind, a, steps)
    if kind.startswith("gradient"):
        g = dtype(1) / np.sqrt(dtype(oracle.DEFAULT_COEF[kind][0]))
        v = dtype(1)
        for _ in range(steps):
            v = dtype(v + g)
        core = tuple(slice(steps + 1, n - steps - 1) for n in shape)
        assert np.all(out[core] == v)
    else:
        assert np.all(out == 1)


def sine_mode(shape, modes, dtype=np.float64):
    grids = np.meshgrid(*[np.arange(n) for n in shape], indexing="ij")
    u = np.ones(shape)
    for g, n, p in zip(grids, shape, modes):
        u = u * np.sin(np.pi * p * g / (n - 1))
    return u.astype(dtype)


def eigenvalue(kind, shape, modes):
    c = oracle.DEFAULT_COEF[kind]
    cs = [np.cos(np.pi * p / (n - 1)) for n, p in zip(shape, modes)]
    if kind == "jacobi2d5":
        return c[0] * (1 + 2 * sum(cs))
    if kind in ("star2d5", "star3d7"):
        return c[0] + 2 * c[1] * sum(cs)
    return c[0] * np.prod([1 + 2 * x for x in cs])


@pytest.mark.parametrize("kind,shape,modes,steps", [
    ("jacobi2d5", (256, 256), (3, 5), 32),
    ("star2d5", (64, 80), (2, 7), 20),
    ("box2d9", (64, 64), (4, 1), 20),
    ("star3d7", (40, 36, 48), (1, 2, 3), 12),
    ("box3d27", (24, 30, 28), (3, 1, 2), 8),
])
def test_dirichlet_sine_mode_decays_by_exact_eigenvalue(kind, shape, modes, steps):
    """The Dirichlet-zero sine mode prod_d sin(pi p_d x_d/(N_d-1)) is an eigenvector of
    every linear class; after T steps it is scaled by lambda^T exactly (closed form)."""
    u = sine_mode(shape, modes)
    lam = eigenvalue(kind, shape, modes)
    got = oracle.run(kind, u, steps)
    exp = u * lam ** steps
    scale = np.max(np.abs(exp))
    assert np.max(np.abs(got - exp)) <= 1e-13 * max(scale, 1e-300) + 1e-14 * steps * np.max(np.abs(u))


@pytest.mark.parametrize("kind", LINEAR)
def test_matches_scipy_correlate_iteration(kind):
    """Each linear class equals T iterations of scipy.ndimage.correlate with the class's
    weights on the interior and untouched Dirichlet boundary cells (library routine)."""
    shape = (33, 47) if oracle.DIMS[kind] == 2 else (13, 17, 19)
    a = stencil_inputs.uniform(shape, seed=3, dtype=np.float64)
    w = kernel_weights(kind)
    ref = a.copy()
    steps = 6
    for _ in range(steps):
        nxt = ref.copy()
        nxt[interior(shape)] = scipy.ndimage.correlate(ref, w, mode="constant")[interior(shape)]
        ref = nxt
    got = oracle.run(kind, a, steps)
    np.testing.assert_allclose(got, ref, rtol=1e-13, atol=1e-14)


@pytest.mark.parametrize("kind", ["star2d5", "box2d9", "star3d7", "box3d27"])
def test_exact_integer_path_counts(kind):
    """With unit coefficients and small integer inputs every fp operation is exact, so the
    oracle must equal the exact integer result M^T x, M the (sparse) iteration matrix
    built from the stencil's offsets with identity rows on the Dirichlet boundary."""
    dims = oracle.DIMS[kind]
    shape = (9, 11) if dims == 2 else (7, 8, 9)
    rng = np.random.default_rng(7)
    x = rng.integers(-3, 4, size=shape).astype(np.int64)
    offs = np.argwhere(kernel_weights(kind) != 0) - 1
    n = x.size
    idx = np.arange(n).reshape(shape)
    rows, cols = [], []
    inner = np.zeros(shape, bool)
    inner[interior(shape)] = True
    for o in offs:
        src = np.roll(idx, shift=tuple(-int(v) for v in o), axis=tuple(range(dims)))
        rows.append(idx[inner]); cols.append(src[inner])
    rows.append(idx[~inner]); cols.append(idx[~inner])
    r = np.concatenate(rows); c = np.concatenate(cols)
    M = scipy.sparse.csr_matrix((np.ones(r.size, np.int64), (r, c)), shape=(n, n))
    steps = 4
    v = x.reshape(-1)
    for _ in range(steps):
        v = M @ v
    coef = (1.0, 1.0) if kind.startswith("star") else (1.0,)
    for dtype in (np.float32, np.float64):
        got = oracle.run(kind, x.astype(dtype), steps, coef=coef)
        assert np.array_equal(got.astype(np.int64).reshape(-1), v)


def test_fdtd_uniform_fields_are_exact_fixpoints():
    """Uniform ex, ey, hz make every difference in the three statements zero."""
    for dtype in (np.float32, np.float64):
        ex = np.full((10, 12), 0.25, dtype); ey = np.full((10, 12), -1.5, dtype)
        hz = np.full((10, 12), 3.0, dtype)
        r = oracle.fdtd(ex, ey, hz, 50)
        assert np.array_equal(r[0], ex) and np.array_equal(r[1], ey) and np.array_equal(r[2], hz)


def test_fdtd_discrete_wave_identity():
    """Eliminating ex, ey from the three statements gives the leapfrog wave equation
    hz^{n+1} - 2 hz^n + hz^{n-1} = (0.7*0.5) * L5(hz^n) on [1,N0-2]x[1,N1-2] for n >= 1,
    L5 the 5-point Laplacian (derivation in DESIGN.md).  Catches sign, index, coefficient
    and domain errors in any of the statements."""
    N = (24, 30)
    ex, ey, hz = stencil_inputs.fields(N, seed=11, n=3, dtype=np.float64)
    hs = [hz]
    state = (ex, ey, hz)
    for _ in range(5):
        state = oracle.fdtd(*state, 1)
        hs.append(state[2])
    ce, ch = oracle.DEFAULT_COEF["fdtd2d"]
    for n in range(1, 5):
        h = hs[n]
        L = np.zeros_like(h)
        L[1:-1, 1:-1] = h[2:, 1:-1] + h[:-2, 1:-1] + h[1:-1, 2:] + h[1:-1, :-2] - 4 * h[1:-1, 1:-1]
        lhs = hs[n + 1] - 2 * h + hs[n - 1]
        np.testing.assert_allclose(lhs[1:-1, 1:-1], (ch * ce) * L[1:-1, 1:-1], atol=1e-13)


@pytest.mark.parametrize("kind,slopes", [("gradient2d", (0.3, -0.7)),
                                          ("gradient3d", (0.5, -0.2, 0.9))])
def test_gradient_ramp_closed_form(kind, slopes):
    """On a linear ramp f = sum_d alpha_d x_d every interior point away from the boundary
    sees (c - nb)^2 = alpha_d^2 twice per axis, so each step adds exactly
    1/sqrt(eps + 2 sum alpha_d^2) (fp64, up to rounding)."""
    dims = len(slopes)
    shape = (16,) * dims
    grids = np.meshgrid(*[np.arange(n, dtype=np.float64) for n in shape], indexing="ij")
    f = sum(a * g for a, g in zip(slopes, grids))
    eps = oracle.DEFAULT_COEF[kind][0]
    inc = 1.0 / np.sqrt(eps + 2 * sum(a * a for a in slopes))
    steps = 3
    got = oracle.run(kind, f, steps)
    core = tuple(slice(steps + 1, n - steps - 1) for n in shape)
    np.testing.assert_allclose(got[core], f[core] + steps * inc, rtol=0, atol=1e-12)


@pytest.mark.parametrize("kind", ["jacobi2d5", "box2d9", "star3d7", "gradient3d"])
@pytest.mark.parametrize("dtype", [np.float32, np.float64])
def test_cone_sampler_matches_full_run(kind, dtype):
    """oracle_points (dependence-cone evaluation used for full-size sampling) is
    bit-identical to the full naive run, including points near the boundary."""
    shape = (37, 29) if oracle.DIMS[kind] == 2 else (15, 13, 17)
    a = stencil_inputs.uniform(shape, seed=5, dtype=dtype)
    steps = 7
    full = oracle.run(kind, a, steps)
    rng = np.random.default_rng(1)
    pts = np.stack([rng.integers(0, n, 40) for n in shape], axis=1)
    pts[0] = [1] * len(shape)
    pts[1] = [n - 2 for n in shape]
    pts[2] = [0] * len(shape)
    got = oracle.points(kind, a, steps, pts)
    assert np.array_equal(got, full[tuple(pts.T)])


def test_openmp_threads_bit_identical():
    """Points inside one time step are independent, so the thread count cannot change
    the result (the bench times the oracle with all host cores)."""
    a = stencil_inputs.uniform((130, 140), seed=2)
    r1 = oracle.run("box2d9", a, 9, nthreads=1)
    r8 = oracle.run("box2d9", a, 9, nthreads=8)
    assert np.array_equal(r1, r8)


def test_zero_steps_and_odd_steps_parity():
    a = stencil_inputs.uniform((20, 21), seed=9)
    assert np.array_equal(oracle.run("star2d5", a, 0), a)
    r3 = oracle.run("star2d5", a, 3)
    r = a
    for _ in range(3):
        r = oracle.run("star2d5", r, 1)
    assert np.array_equal(r3, r)
