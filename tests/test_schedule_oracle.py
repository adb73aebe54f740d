"""Pins of the schedule oracle (oracle/schedule.py) against the paper's own statements and
brute-force enumeration: exactly-once coverage, every RAW/WAR/WAW dependence respected,
no dependence inside one phase across tiles, the printed Fig. 6 instance, the printed
worked example, the printed tile-size formula and the eq. (1) threshold."""
from fractions import Fraction as Fr

import pytest

from oracle import schedule as S


def test_paper_example_slopes_and_w0_bound():
    """Sec. 3.3.2 example A[t][i] = f(A[t-2][i-2], A[t-1][i+2]) has distance vectors
    {(1,-2); (2,2)} -> delta0 = 1, delta1 = 2 (Fig. 3) and with h=2
    eq. (1) gives 'w0 >= 1'."""
    d0, d1 = S.slopes([(1, -2), (2, 2)])
    assert (d0, d1) == (1, 2)
    assert S.w0_lower_bound(d0, d1, 2) == 1


def _check_explicit(distances, hx, T=24, N=60):
    """Coverage + order for a 1-D program given by explicit flow-distance vectors."""
    sched = {}
    bad = 0
    for t in range(T):
        for s in range(N):
            tl = S.hex_tile(hx, t, s)
            if len(tl) != 1:
                bad += 1
                continue
            T_, p, S0, a, b = tl[0]
            sched[(t, s)] = ((T_, p), S0, a)
    viol = 0
    for (t, s), (tp, S0, a) in sched.items():
        for dt, ds in distances:
            src = (t - dt, s - ds)
            if src in sched:
                tps, S0s, as_ = sched[src]
                if not (tps < tp or (tps == tp and S0s == S0 and as_ < a)):
                    viol += 1
    return bad, viol


@pytest.mark.parametrize("w0", [1, 2, 3])
def test_paper_example_schedule_valid_for_w0_at_bound(w0):
    """The example's hexagonal schedule (h=2, Fig. 4) covers every point once and respects
    both flow dependences for w0 >= 1 (eq. (1))."""
    hx = S.Hex(Fr(1), Fr(2), 2, w0)
    assert _check_explicit([(1, -2), (2, 2)], hx) == (0, 0)


def test_paper_example_below_bound_fails():
    """w0 = 0 < eq. (1)'s bound: the subtraction of Fig. 4 is not convex and the schedule
    breaks (reproduces the brown dependence vector argument)."""
    hx = S.Hex(Fr(1), Fr(2), 2, 0)
    bad, viol = _check_explicit([(1, -2), (2, 2)], hx)
    assert bad + viol > 0


def test_literal_eq3_breaks_coverage_when_slopes_differ():
    """Reading R1: the extracted eq. (3) (floor(delta1 h) in the phase-0 numerator) does not
    tile the plane when delta0 != delta1; floor(delta0 h) does."""
    hx = S.Hex(Fr(1), Fr(2), 2, 1)
    bad_lit = sum(len(S.hex_tile(hx, t, s, literal_eq3=True)) != 1 for t in range(30) for s in range(60))
    bad_fix = sum(len(S.hex_tile(hx, t, s)) != 1 for t in range(30) for s in range(60))
    assert bad_lit > 0 and bad_fix == 0


@pytest.mark.parametrize("h,w0", [(0, 0), (1, 0), (1, 3), (2, 7), (3, 15), (4, 2)])
def test_full_tile_point_count_matches_paper(h, w0):
    """Sec. 3.7: a tile with delta0 = delta1 = 1 has
    2(1 + 2h + h^2 + w0(h+1)) points per classical column."""
    pts, _, _ = S.tile_in_out_counts(S.Hex(Fr(1), Fr(1), h, w0))
    assert pts == 2 * (1 + 2 * h + h * h + w0 * (h + 1))


@pytest.mark.parametrize("h,w0", [(1, 3), (2, 7), (3, 7), (3, 15), (5, 8)])
def test_in_out_traffic_closed_form(h, w0):
    """Brute-force In/Out sets of a full radius-1 hexagon equal the closed forms used by
    the roofline model: In = w0+4h+5, Out = w0+4h+3 values per column."""
    pts, n_in, n_out = S.tile_in_out_counts(S.Hex(Fr(1), Fr(1), h, w0))
    assert (n_in, n_out) == (w0 + 4 * h + 5, w0 + 4 * h + 3)


@pytest.mark.parametrize("h,w0,w1", [(1, 0, 3), (2, 3, 4), (3, 1, 5)])
def test_fig6_equals_general_schedule_for_unit_slopes(h, w0, w1):
    """Fig. 6 is the printed instance of the general schedule for +-1
    distances: every phase-0 point maps to the same tuple, every phase-1 point is
    rejected by Fig. 6's constraints."""
    hx = S.Hex(Fr(1), Fr(1), h, w0)
    for t in range(3 * (2 * h + 2)):
        for s0 in range(-3, 40):
            for s1 in range(-2, 12):
                full = S.hybrid(hx, [Fr(1)], [w1], t, (s0, s1))
                f6 = S.fig6(h, w0, [w1], t, (s0, s1))
                if full[1] == 0:
                    assert f6 == full
                else:
                    assert f6 is None


@pytest.mark.parametrize("offsets,N,steps,h,w0,w1", [
    (S.STAR2D5, (26, 13), 14, 1, 0, 3),
    (S.STAR2D5, (30, 17), 13, 3, 5, 6),
    (S.STAR2D5, (23, 11), 11, 2, 2, 4),
    (S.BOX2D9, (26, 13), 12, 2, 3, 5),
    (S.BOX2D9, (25, 12), 12, 0, 0, 2),
])
def test_hybrid_schedule_valid_2d(offsets, N, steps, h, w0, w1):
    """Exactly-once coverage and all memory-based dependences (RAW, WAR, WAW of the
    ping-pong layout) respected by [T,p,S0,S1,t'] (Sec. 3.6)."""
    prog = S.single_statement(offsets)
    dv = S.distance_vectors(S.dependences(prog, N, 4))
    d0, d1 = S.slopes([(d[0], d[1]) for d in dv])
    _, d1j = S.slopes([(d[0], d[2]) for d in dv])
    assert (d0, d1, d1j) == (1, 1, 1)
    r = S.check_schedule(prog, N, steps, S.Hex(d0, d1, h, w0), [d1j], [w1])
    assert r["coverage"] == r["order"] == r["same_phase"] == r["same_step"] == 0, r


@pytest.mark.parametrize("offsets,h,w0,w", [(S.STAR3D7, 1, 1, (3, 4)), (S.BOX3D27, 1, 0, (2, 3))])
def test_hybrid_schedule_valid_3d(offsets, h, w0, w):
    prog = S.single_statement(offsets)
    N = (14, 7, 8)
    r = S.check_schedule(prog, N, 8, S.Hex(Fr(1), Fr(1), h, w0), [Fr(1), Fr(1)], list(w))
    assert r["coverage"] == r["order"] == r["same_phase"] == r["same_step"] == 0, r


def test_radius2_below_eq1_bound_breaks():
    """Radius 2 along s0 has delta = 2; eq. (1) requires w0 >= 1.  w0 = 0 must fail and
    w0 = 1 must pass (the eq. (1) threshold reproduced by enumeration)."""
    offs = [(0, 0), (-2, 0), (2, 0), (-1, 0), (1, 0), (0, 1), (0, -1)]
    prog = S.single_statement(offs)
    N = (28, 8)
    assert S.w0_lower_bound(Fr(2), Fr(2), 2) == 1
    bad = S.check_schedule(prog, N, 12, S.Hex(Fr(2), Fr(2), 2, 0), [Fr(1)], [4])
    good = S.check_schedule(prog, N, 12, S.Hex(Fr(2), Fr(2), 2, 1), [Fr(1)], [4])
    assert bad["coverage"] + bad["order"] + bad["same_phase"] + bad["same_step"] > 0
    assert good["coverage"] == good["order"] == good["same_phase"] == good["same_step"] == 0


def test_fdtd_dependence_slopes():
    """FDTD-2D with tau = 3t + k (Sec. 3.2) and in-place fields: along i delta0 = 1,
    delta1 = 1/2 (rational -> denominators d0 = 1, d1 = 2 in eqs. (10), (12)); along j the
    classical slope delta1_j = 1 (reading R14)."""
    dv = S.distance_vectors(S.dependences(S.FDTD2D, (9, 10), 4))
    assert S.slopes([(d[0], d[1]) for d in dv]) == (1, Fr(1, 2))
    assert S.slopes([(d[0], d[2]) for d in dv])[1] == 1


@pytest.mark.parametrize("h,w0,w1", [(2, 0, 4), (2, 1, 3), (3, 2, 5), (5, 3, 4), (4, 1, 6)])
def test_fdtd_hybrid_schedule_valid(h, w0, w1):
    """The corrected schedule is valid for the three-statement in-place FDTD kernel,
    including h+1 not a multiple of 3 (the multiple only makes tiles uniform, reading R14)."""
    hx = S.Hex(Fr(1), Fr(1, 2), h, w0)
    assert w0 >= S.w0_lower_bound(hx.d0, hx.d1, h)
    r = S.check_schedule(S.FDTD2D, (22, 11), 8, hx, [Fr(1)], [w1])
    assert r["coverage"] == r["order"] == r["same_phase"] == r["same_step"] == 0, r


@pytest.mark.parametrize("offsets", [S.STAR3D7, S.BOX3D27])
def test_larger_skew_and_translation_stay_valid(offsets):
    """The 3D kernel skews x by 4 per level (>= delta1_x = 1) and translates x tiles by +1
    (Sec. 4.2.3's translation offset): still exactly-once and
    dependence-respecting (reading R16)."""
    prog = S.single_statement(offsets)
    N = (12, 7, 19)
    r = S.check_schedule(prog, N, 7, S.Hex(Fr(1), Fr(1), 1, 1), [Fr(1), Fr(4)], [3, 8],
                         trans=[0, 1])
    assert r["coverage"] == r["order"] == r["same_phase"] == r["same_step"] == 0, r


# ---- pins of the dependence simulator itself (oracle/schedule.py::dependences) ----------
# The sets below are fixed by the paper's programs and the memory layout, derived by hand
# (no call into the code under test): a plausible slip in the simulator (a dropped WAR or
# WAW edge, a wrong parity slot, a reversed offset) changes one of them.

def test_dependences_fig1_pingpong_exact_set():
    """Fig. 1: A[(t+1)%2][i][j] = f(A[t%2][i+-1][j], A[t%2][i][j+-1],
    A[t%2][i][j]).  RAW: the value read at offset o was written one step earlier at s+o:
    (1, -o).  WAR: the location A[t%2][s+o] read at step t is overwritten at step t+1 by the
    instance at s+o: (1, o).  WAW: A[(t+1)%2][s] is rewritten at step t+2: (2, 0)."""
    prog = S.single_statement(S.STAR2D5)
    typed = S.typed_distance_vectors(S.dependences(prog, (7, 8), 4, typed=True))
    star = {(1, 0, 0), (1, 1, 0), (1, -1, 0), (1, 0, 1), (1, 0, -1)}
    assert typed["RAW"] == star
    assert typed["WAR"] == star
    assert typed["WAW"] == {(2, 0, 0)}
    assert S.distance_vectors(S.dependences(prog, (7, 8), 4)) == star | {(2, 0, 0)}


def test_dependences_one_sided_stencil_separates_raw_from_war():
    """A one-sided ping-pong stencil A'[s] = f(A[s], A[s+1]): RAW distances (1, -o) =
    {(1,0), (1,-1)}, WAR distances (1, +o) = {(1,0), (1,1)}, WAW (2,0).  Dropping the WAR
    edges loses (1, 1); dropping WAW loses (2, 0); swapping RAW/WAR flips the signs."""
    prog = S.single_statement([(0,), (1,)])
    typed = S.typed_distance_vectors(S.dependences(prog, (12,), 5, typed=True))
    assert typed == {"RAW": {(1, 0), (1, -1)}, "WAR": {(1, 0), (1, 1)}, "WAW": {(2, 0)}}
    assert S.distance_vectors(S.dependences(prog, (12,), 5)) == {(1, 0), (1, -1), (1, 1), (2, 0)}
    # the cone these span: delta0 = 1 (from (1, 1), a WAR edge), delta1 = 1 (RAW (1, -1))
    assert S.slopes(S.distance_vectors(S.dependences(prog, (12,), 5))) == (1, 1)


def test_dependences_paper_example_through_simulator():
    """The example of Sec. 3.3.2, A[t][i] = f(A[t-2][i-2], A[t-1][i+2]) with a time-expanded
    array, has exactly the distance vectors {(1,-2); (2,2)}: RAW only,
    since no location is reused.  Fed through the memory simulator, then Fig. 3's slopes."""
    prog = S.expanded_program([(-2, (-2,)), (-1, (2,))], lo=(2,), hi=(-2,))
    typed = S.typed_distance_vectors(S.dependences(prog, (16,), 7, typed=True))
    assert typed == {"RAW": {(1, -2), (2, 2)}, "WAR": set(), "WAW": set()}
    assert S.slopes(S.distance_vectors(S.dependences(prog, (16,), 7))) == (1, 2)


def test_dependences_fdtd_exact_sets():
    """FDTD-2D in place with tau = 3t+k (ey k=0, ex k=1, hz k=2; Sec. 3.2),
    derived by hand from the three statements (reading R9):
      RAW  ey<-hz(t-1): (1,0,0), (1,1,0); ex<-hz(t-1): (2,0,0), (2,0,1);
           hz<-ex(t): (1,0,-1), (1,0,0); hz<-ey(t): (2,-1,0), (2,0,0); self: (3,0,0)
      WAR  hz(t) overwrites what ey(t) read: (2,0,0), (2,-1,0); what ex(t) read: (1,0,0),
           (1,0,-1); ex(t+1) overwrites what hz(t) read: (2,0,1), (2,0,0); ey(t+1): (1,1,0),
           (1,0,0)
      WAW  every field once per step: (3,0,0)"""
    typed = S.typed_distance_vectors(S.dependences(S.FDTD2D, (7, 8), 4, typed=True))
    assert typed["RAW"] == {(1, 0, 0), (1, 1, 0), (2, 0, 0), (2, 0, 1), (1, 0, -1), (2, -1, 0), (3, 0, 0)}
    assert typed["WAR"] == {(2, 0, 0), (2, -1, 0), (1, 0, 0), (1, 0, -1), (2, 0, 1), (1, 1, 0)}
    assert typed["WAW"] == {(3, 0, 0)}
