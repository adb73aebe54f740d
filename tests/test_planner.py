"""Host-side tests of the product planner (libhexstencil.so: dependence analysis a1, tile
validation a2, launch table a3) against the schedule oracle, plus the C-ABI surface.
No GPU needed: planning never touches the device."""
import ctypes
import os
import re
from fractions import Fraction as Fr

import numpy as np
import pytest

import oracle
from oracle import schedule as S
from paper_conf_cgo_grosserchsv14_b200 import Plan, Stencil, StencilError
from paper_conf_cgo_grosserchsv14_b200 import _lib

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))

PROGRAMS = {
    "jacobi2d5": S.single_statement(S.STAR2D5), "star2d5": S.single_statement(S.STAR2D5),
    "gradient2d": S.single_statement(S.STAR2D5), "box2d9": S.single_statement(S.BOX2D9),
    "star3d7": S.single_statement(S.STAR3D7), "gradient3d": S.single_statement(S.STAR3D7),
    "box3d27": S.single_statement(S.BOX3D27), "fdtd2d": S.FDTD2D,
}


def test_library_exports_every_header_symbol():
    """The C-ABI library loads (no GPU needed) and exports every function include/stencil.h
    declares."""
    hdr = open(os.path.join(ROOT, "include", "stencil.h")).read()
    declared = set(re.findall(r"^(?:stencil_status|const char \*|int)\s*(stencil_\w+)\s*\(", hdr, re.M))
    assert declared == set(_lib.SYMBOLS), declared ^ set(_lib.SYMBOLS)
    L = _lib.lib()
    for name in declared:
        assert hasattr(L, name)
    assert L.stencil_abi_version() == 1


@pytest.mark.parametrize("kind", sorted(PROGRAMS))
def test_dependence_distances_match_bruteforce(kind):
    """a1: the closed-form distance set equals a brute-force simulation of the original
    program's memory accesses (oracle/schedule.py::dependences)."""
    dims = oracle.DIMS[kind]
    st = Stencil(kind, (9,) * dims)
    N = (7, 8) if dims == 2 else (6, 6, 7)
    exp = S.distance_vectors(S.dependences(PROGRAMS[kind], N, 4))
    assert set(st.dependences()) == exp


@pytest.mark.parametrize("kind,h,w0", [("star2d5", 3, 10), ("box2d9", 2, 3), ("fdtd2d", 5, 3),
                                        ("fdtd2d", 2, 0), ("star3d7", 2, 7), ("gradient2d", 1, 0)])
def test_slopes_and_hexagon_match_oracle(kind, h, w0):
    """a2: delta0/delta1 (Fig. 3), F0/F1, box size and the hexagon rows of constraints
    (6)-(13) equal the oracle's exact-arithmetic evaluation."""
    dims = oracle.DIMS[kind]
    plan = Plan(Stencil(kind, (40,) * dims), 10, h=h, w0=w0, executor="generic")
    info = plan.info
    dv = S.distance_vectors(S.dependences(PROGRAMS[kind], (7, 8) if dims == 2 else (6, 6, 7), 4))
    d0, d1 = S.slopes([(d[0], d[1]) for d in dv])
    assert (Fr(info["delta0_num"], info["delta0_den"]), Fr(info["delta1_num"], info["delta1_den"])) == (d0, d1)
    hx = S.Hex(d0, d1, h, w0)
    assert (info["H"], info["W"], info["F0"], info["F1"]) == (hx.height, hx.width, hx.F0, hx.F1)
    lo, hi = plan.hexagon()
    assert list(zip(lo, hi)) == S.hexagon_rows(hx)


def test_traffic_model_counts():
    """Plan info carries the per-column tile counts used by the roofline model; they match
    the brute-force In/Out sets (w0+4h+5 / w0+4h+3 for radius 1)."""
    for h, w0 in [(3, 10), (3, 15), (2, 7)]:
        i = Plan(Stencil("star2d5", (64, 64)), 8, h=h, w0=w0, executor="generic").info
        pts, n_in, n_out = S.tile_in_out_counts(S.Hex(Fr(1), Fr(1), h, w0))
        assert (i["tile_points"], i["tile_in"], i["tile_out"]) == (pts, n_in, n_out)


def _oracle_sched(kind, plan, tau, s):
    info = plan.info
    hx = S.Hex(Fr(info["delta0_num"], info["delta0_den"]), Fr(info["delta1_num"], info["delta1_den"]),
               info["h"], info["w0"])
    dims = len(s)
    ncls = dims - 1
    return S.hybrid(hx, [Fr(x) for x in info["delta_cls"][:ncls]], info["w"][:ncls], tau, s,
                    info["trans_cls"][:ncls])


@pytest.mark.parametrize("kind,N,T,h,w0,w", [
    ("star2d5", (23, 19), 9, 1, 0, (5, 0)),
    ("star2d5", (40, 30), 12, 3, 10, (7, 0)),
    ("box2d9", (31, 17), 7, 2, 3, (4, 0)),
    ("fdtd2d", (26, 14), 6, 5, 3, (6, 0)),
    ("fdtd2d", (20, 9), 5, 2, 0, (3, 0)),
    ("star3d7", (15, 9, 10), 6, 1, 2, (3, 4)),
])
def test_schedule_of_matches_oracle_hybrid(kind, N, T, h, w0, w):
    """a3: the product's [T, p, S0, S1..Sn, t', s'0..s'n] of every instance equals the
    oracle's literal eqs. (2)-(17) (Sec. 3.6)."""
    plan = Plan(Stencil(kind, N), T, h=h, w0=w0, w=list(w) + [0], executor="generic")
    prog = PROGRAMS[kind]
    for tau, s, st, t in S.instances(prog, N, T):
        assert plan.schedule_of(tau, s) == _oracle_sched(kind, plan, tau, s), (tau, s)


def _enumerate_launch_table(plan, N):
    """Expand the launch table into the set of (tau, s0) row instances it executes."""
    info = plan.info
    lo, hi = plan.hexagon()
    W = info["W"]
    seen = {}
    for idx, ln in enumerate(plan.launches()):
        for S0 in range(ln["S0_lo"], ln["S0_hi"] + 1):
            for a in range(ln["a_lo"], ln["a_hi"] + 1):
                tau = ln["tau0"] + a
                for b in range(lo[a], hi[a] + 1):
                    s0 = S0 * W + b - ln["row_off"]
                    seen.setdefault((tau, s0), []).append((idx, S0))
    return seen


@pytest.mark.parametrize("kind,N,T,h,w0", [("star2d5", (37, 20), 13, 3, 2), ("star2d5", (50, 9), 8, 1, 0),
                                            ("box2d9", (29, 12), 11, 2, 5), ("fdtd2d", (33, 10), 7, 5, 2),
                                            ("star3d7", (21, 6, 6), 5, 2, 1)])
def test_launch_table_covers_each_row_instance_once(kind, N, T, h, w0):
    """Every (tau, s0) of the statement domains appears in exactly one launch entry and
    hexagon, and the launch of each instance is the oracle's (T, p) in order."""
    plan = Plan(Stencil(kind, N), T, h=h, w0=w0, executor="generic")
    seen = _enumerate_launch_table(plan, N)
    launches = plan.launches()
    prog = PROGRAMS[kind]
    want = set()
    for tau, s, st, t in S.instances(prog, N, T):
        want.add((tau, s[0]))
    got = {k for k in seen if k in want}
    assert got == want
    for key in want:
        assert len(seen[key]) == 1, key
        idx, S0 = seen[key][0]
        sched = plan.schedule_of(key[0], (key[1],) + (1,) * (len(N) - 1))
        assert (launches[idx]["T"], launches[idx]["phase"], S0) == sched[:3]
    order = [(l["T"], l["phase"]) for l in launches]
    assert order == sorted(order) and len(set(order)) == len(order)


def _cpu_execute_plan(plan, grid, coef):
    """Test tooling: execute the plan's launch table point by point on the CPU in the
    schedule's order (T, p) -> S0 -> S1 -> t' (star2d5 expression, float32 numpy scalars),
    to show the order reproduces the naive loop bit for bit (reordering invariance)."""
    info = plan.info
    lo, hi = plan.hexagon()
    W, w1 = info["W"], info["w"][0]
    N0, N1 = grid.shape
    buf = [grid.copy(), grid.copy()]
    c0, c1 = np.float32(coef[0]), np.float32(coef[1])
    for ln in plan.launches():
        for S0 in range(ln["S0_lo"], ln["S0_hi"] + 1):
            for S1 in range(-2, (N1 + 2 * info["H"]) // w1 + 2):
                for a in range(ln["a_lo"], ln["a_hi"] + 1):
                    tau = ln["tau0"] + a
                    src, dst = buf[tau % 2], buf[(tau + 1) % 2]
                    for b in range(lo[a], hi[a] + 1):
                        i = S0 * W + b - ln["row_off"]
                        if not 1 <= i <= N0 - 2:
                            continue
                        for j in range(S1 * w1 - a, S1 * w1 - a + w1):
                            if 1 <= j <= N1 - 2:
                                dst[i, j] = c0 * src[i, j] + c1 * (((src[i - 1, j] + src[i + 1, j]) + src[i, j - 1]) + src[i, j + 1])
    return buf[plan.T_steps % 2]


@pytest.mark.parametrize("N,T,h,w0,w1", [((19, 17), 9, 1, 1, 4), ((24, 13), 11, 3, 2, 5)])
def test_cpu_execution_of_launch_table_is_bit_identical_to_oracle(N, T, h, w0, w1):
    import stencil_inputs

    grid = stencil_inputs.uniform(N, seed=4)
    plan = Plan(Stencil("star2d5", N), T, h=h, w0=w0, w=[w1, 0, 0], executor="generic")
    got = _cpu_execute_plan(plan, grid, oracle.DEFAULT_COEF["star2d5"])
    assert np.array_equal(got, oracle.run("star2d5", grid, T))


def test_error_paths():
    with pytest.raises(StencilError) as e:
        Plan(Stencil("box2d9", (32, 32)), 4, h=2, w0=0, hex_dim=1)
    assert e.value.status == 1  # innermost dim cannot be hexagonal
    # radius-1 stencils need w0 >= 0 (eq. 1); a bad kind / dims / coefficient count fail
    with pytest.raises(StencilError):
        Stencil("star3d7", (8, 8))
    with pytest.raises(StencilError):
        Stencil("star2d5", (8, 8), coefficients=[1.0])
    with pytest.raises(StencilError):
        Stencil("star2d5", (2, 8))
    with pytest.raises(StencilError):
        Stencil("star2d5", (8, 8), offsets=[(0, 0), (1, 0)])
    Stencil("star2d5", (8, 8), offsets=[(0, 1), (0, 0), (1, 0), (-1, 0), (0, -1)])
    with pytest.raises(StencilError):
        Plan(Stencil("star2d5", (8, 8)), -1)
    with pytest.raises(StencilError):
        Plan(Stencil("star2d5", (8, 8)), 4, h=40, w0=1)  # 2h+2 > 64 levels
    L = _lib.lib()
    assert L.stencil_destroy(None) == 0
    # T mismatch is rejected before any CUDA call
    p = Plan(Stencil("star2d5", (8, 8)), 4, executor="generic")
    dummy = (ctypes.c_void_p * 1)(16)
    assert L.stencil_run(p._h, dummy, dummy, 5, None) == 1
    assert b"T_steps" in L.stencil_last_error()


def test_eq1_bound_enforced_for_rational_slopes():
    """FDTD (delta = 1, 1/2) admits w0 = 0 for every h (eq. 1); the worked example's bound
    is covered by the oracle tests."""
    for h in range(0, 7):
        Plan(Stencil("fdtd2d", (20, 20)), 3, h=h, w0=0, executor="generic")


def test_naive_and_auto_executor_selection():
    p = Plan(Stencil("star2d5", (64, 64)), 8, executor="naive")
    assert p.info["executor"] == 2 and p.info["n_launches"] == 8
    p = Plan(Stencil("star2d5", (64, 64)), 8)
    assert p.info["fast_kernel"] == 1  # a compiled variant, the tile model's choice for this grid
    p = Plan(Stencil("star2d5", (8192, 8192)), 8)
    assert p.info["fast_kernel"] == 1 and (p.info["h"], p.info["w0"]) == (2, 7)  # tile model, round 2
    p = Plan(Stencil("star2d5", (64, 64)), 8, h=2, w0=2)   # no specialised instantiation
    assert p.info["fast_kernel"] == 0
    assert p.workspace_bytes >= 64 * 64 * 4
    assert Plan(Stencil("fdtd2d", (64, 64)), 8).workspace_bytes == 0
