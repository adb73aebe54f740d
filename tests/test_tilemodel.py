"""Host-side tests of the tile-size model (include/stencil.h stencil_tile_model, csrc/tilemodel.cpp:
Sec. 3.7's load-to-compute ratio, with the instruction-cache and CTA-count terms)
and of the planner on general linear stencils (any access set / radius: general delta)."""
import ctypes
from fractions import Fraction as Fr

import pytest

from oracle import schedule as S
from paper_conf_cgo_grosserchsv14_b200 import Plan, Stencil, _lib
from paper_conf_cgo_grosserchsv14_b200._lib import TileEval, check, lib


def _eval(st, h, w0, family, hex_dim=0):
    e = TileEval()
    check(lib().stencil_tile_model(st._h, h, w0, hex_dim, family, ctypes.byref(e)))
    return e


# best (h, w0) measured on B200 among each class's compiled variants (profiles/round1/tile_sweep_*,
# round 2: profiles/round2/tile_sweep_2d.txt -- star2d5 moved to (2, 7) with the select-free body)
MEASURED_BEST = [("star2d5", (8192, 8192), 1, (2, 7)), ("box2d9", (8192, 8192), 1, (2, 7)),
                 ("gradient2d", (8192, 8192), 1, (1, 1)), ("star3d7", (512, 512, 512), 2, (3, 7))]


@pytest.mark.parametrize("kind,ext,family,best", MEASURED_BEST)
def test_model_picks_the_measured_best_tile(kind, ext, family, best):
    st = Stencil(kind, ext)
    assert _eval(st, *best, family).selected == 1
    info = Plan(st, 64).info  # the planner's automatic tile is the model's choice
    assert (info["h"], info["w0"]) == best


@pytest.mark.parametrize("h,w0", [(1, 3), (2, 7), (3, 7), (3, 15), (4, 5)])
def test_load_to_compute_term_is_the_exact_hexagon_count(h, w0):
    """B = 4 (In + Out) / points of the brute-force hexagon (oracle/schedule.py), i.e. the closed
    form 4 (w0 + 4h + 4) / ((h+1)(h+w0+1)) for unit slopes."""
    e = _eval(Stencil("star2d5", (4096, 4096)), h, w0, 0)
    pts, n_in, n_out = S.tile_in_out_counts(S.Hex(Fr(1), Fr(1), h, w0))
    assert (e.points, e.in_, e.out) == (pts, n_in, n_out)
    assert abs(e.bytes_per_update - 4 * (w0 + 4 * h + 4) / ((h + 1) * (h + w0 + 1))) < 1e-12


def test_code_and_wave_terms():
    st = Stencil("star2d5", (8192, 8192))
    small, big = _eval(st, 2, 7, 1), _eval(st, 4, 5, 1)
    assert small.code_eff == 1.0 and big.code_eff < 1.0  # the larger unrolled body overflows
    assert small.body_bytes < big.body_bytes
    e = _eval(st, 3, 5, 1)  # W = 18: 456 hexagons on 444 slots -> two waves
    waves = -(-e.ctas // e.slots)
    assert waves == 2 and abs(e.wave_eff - e.ctas / (waves * e.slots)) < 1e-12
    assert _eval(st, 2, 7, 0).code_eff == 1.0  # generic kernel: rolled loops, no code term


STAR2D_R2 = [(0, 0), (-1, 0), (1, 0), (0, -1), (0, 1), (-2, 0), (2, 0), (0, -2), (0, 2)]
UPWIND2D = [(0, 0), (0, -1), (0, -2), (-1, 0)]


def test_linear_stencil_dependences_match_bruteforce():
    """a1 for a general access set: the closed-form distance set equals the memory simulator's."""
    for offs in (STAR2D_R2, UPWIND2D):
        st = Stencil("linear", (12, 13), offsets=offs, coefficients=[0.1] * len(offs))
        exp = S.distance_vectors(S.dependences(S.single_statement(offs), (9, 10), 4))
        assert set(st.dependences()) == exp


def test_linear_radius2_plan_follows_eq1_and_the_schedule_oracle():
    """Radius 2 -> delta0 = delta1 = 2, eq. (1) needs w0 >= 1; the planner's schedule equals the
    oracle's literal eqs. (2)-(17) for every instance of a small window."""
    st = Stencil("linear", (40, 23), offsets=STAR2D_R2, coefficients=[0.1] * 9)
    with pytest.raises(_lib.StencilError):
        Plan(st, 10, h=2, w0=0, executor="generic")
    plan = Plan(st, 10, h=2, w0=1, executor="generic")
    info = plan.info
    assert (info["delta0_num"], info["delta1_num"], info["delta_cls"][0]) == (2, 2, 2)
    hx = S.Hex(Fr(2), Fr(2), 2, 1)
    assert list(zip(*plan.hexagon())) == S.hexagon_rows(hx)
    w1 = info["w"][0]
    for t in range(0, 12):
        for s0 in range(0, 40, 3):
            for s1 in range(0, 23, 4):
                exp = S.hybrid(hx, [Fr(2)], [w1], t, (s0, s1))
                assert plan.schedule_of(t, (s0, s1)) == exp


def test_linear_auto_tile_from_the_model():
    st = Stencil("linear", (2048, 2048), offsets=STAR2D_R2, coefficients=[0.1] * 9)
    info = Plan(st, 32).info
    e = _eval(st, info["h"], info["w0"], 0)
    assert e.selected == 1 and info["executor"] == 1  # generic executor (no fast kernel)
    assert info["w0"] >= 1  # eq. (1) for delta = 2
