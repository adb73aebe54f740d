"""Schedule oracle: the hybrid hexagonal/classical schedule of Grosser et al. (CGO'14),
written out literally from Sec. 3 of /root/reference/PAPER.md in exact rational
arithmetic, plus the brute-force checks that pin it.

TEST INFRASTRUCTURE ONLY -- imported by tests/ (and nothing in the product path).
It shares no code with the product's C++ planner (paper_conf_cgo_grosserchsv14_b200/
csrc/plan.cpp); tests compare the two.

Contents, in the paper's order and notation:
  * memory-based dependences of the canonical schedule [k*t+i, s] (Sec. 3.1-3.2,
    PAPER.md:253-299), by brute-force simulation of the original program order
    (Feautrier-style dataflow on a small grid -- `dependences`);
  * cone slopes delta0, delta1 (Sec. 3.3.2, Fig. 3) -- `slopes`;
  * the width bound, eq. (1) -- `w0_lower_bound`;
  * the two-phase hexagonal tile schedule, eqs. (2)-(5), with the
    phase-0 numerator read as floor(delta0*h) (reading R1: the extracted
    eq. (3) shows floor(delta1*h), which fails exact coverage whenever delta0 != delta1;
    `hex_tile_literal_eq3` keeps the extracted text so a test can show that) --
    `hex_tile`;
  * the hexagon constraints (6), (7), (8), (10), (12), (13) in local coordinates
     -- `in_hexagon`;
  * classical tiling eqs. (14)-(16) and the intra-tile schedule eq. (17)
     -- `classical`;
  * the hybrid map [t, s0..sn] -> [T, p, S0..Sn, t', s'0..s'n] (Sec. 3.6)
    -- `hybrid`; and Fig. 6, the paper's printed instance for +-1 distances -- `fig6`;
  * the validity check used by the tests (exactly-once coverage, every dependence
    respected, no dependence inside one (T, p) across S0 or inside one
    (T, p, S0, S1..Sn, t')) -- `check_schedule`.
"""
from __future__ import annotations

from dataclasses import dataclass
from fractions import Fraction as Fr
from itertools import product
from math import floor
from typing import Dict, Iterable, List, Optional, Sequence, Tuple

# --------------------------------------------------------------------------------------
# Programs: an outer time loop around k >= 1 perfect nests without carried dependences
# (Sec. 3.2).  A statement writes one array at offset 0 and reads a
# list of (array, offset) pairs.  `pingpong=True` is Fig. 1's A[(t+1)%2] = f(A[t%2])
# layout; otherwise arrays are updated in place (FDTD).
# --------------------------------------------------------------------------------------


@dataclass(frozen=True)
class Statement:
    write: str
    reads: Tuple[Tuple[str, Tuple[int, ...]], ...]
    lo: Tuple[int, ...]  # domain lower bound per spatial dim, relative to 0
    hi: Tuple[int, ...]  # domain upper bound per spatial dim, relative to N (exclusive): N + hi
    versions: Tuple[int, ...] = ()  # time-expanded layout only: read i reads A[t + versions[i]]


@dataclass(frozen=True)
class Program:
    dims: int
    statements: Tuple[Statement, ...]
    pingpong: bool
    expanded: bool = False  # time-expanded arrays A[t][s]: no location is ever reused


def single_statement(offsets: Sequence[Tuple[int, ...]]) -> Program:
    """A[(t+1)%2][s] = f(A[t%2][s+o] for o in offsets) over the interior [1, N-2]^d (Fig. 1)."""
    dims = len(offsets[0])
    st = Statement("A", tuple(("A", tuple(o)) for o in offsets), (1,) * dims, (-1,) * dims)
    return Program(dims, (st,), True)


STAR2D5 = [(0, 0), (-1, 0), (1, 0), (0, -1), (0, 1)]
BOX2D9 = [(di, dj) for di in (-1, 0, 1) for dj in (-1, 0, 1)]
STAR3D7 = [(0, 0, 0), (-1, 0, 0), (1, 0, 0), (0, -1, 0), (0, 1, 0), (0, 0, -1), (0, 0, 1)]
BOX3D27 = [(a, b, c) for a in (-1, 0, 1) for b in (-1, 0, 1) for c in (-1, 0, 1)]

# FDTD-2D (Table 3; PolyBench form, reading R9):
#   ey[i][j] = f(ey[i][j], hz[i][j], hz[i-1][j])                 i in [1, N0),   j in [0, N1)
#   ex[i][j] = f(ex[i][j], hz[i][j], hz[i][j-1])                 i in [0, N0),   j in [1, N1)
#   hz[i][j] = f(hz[i][j], ex[i][j+1], ex[i][j], ey[i+1][j], ey[i][j])
#                                                                i in [0, N0-1), j in [0, N1-1)
FDTD2D = Program(
    2,
    (
        Statement("ey", (("ey", (0, 0)), ("hz", (0, 0)), ("hz", (-1, 0))), (1, 0), (0, 0)),
        Statement("ex", (("ex", (0, 0)), ("hz", (0, 0)), ("hz", (0, -1))), (0, 1), (0, 0)),
        Statement(
            "hz",
            (("hz", (0, 0)), ("ex", (0, 1)), ("ex", (0, 0)), ("ey", (1, 0)), ("ey", (0, 0))),
            (0, 0),
            (-1, -1),
        ),
    ),
    False,
)


def expanded_program(reads: Sequence[Tuple[int, Tuple[int, ...]]], lo: Sequence[int],
                     hi: Sequence[int]) -> Program:
    """A[t][s] = f(A[t + dt][s + ds] for (dt, ds) in reads) with a time-expanded array (every
    version has its own memory), e.g. the example of Sec. 3.3.2,
    A[t][i] = f(A[t-2][i-2], A[t-1][i+2])."""
    dims = len(reads[0][1])
    st = Statement("A", tuple(("A", tuple(o)) for _, o in reads), tuple(lo), tuple(hi),
                   tuple(dt for dt, _ in reads))
    return Program(dims, (st,), False, True)


def instances(prog: Program, N: Sequence[int], steps: int):
    """Statement instances in the ORIGINAL program order, as (tau, s) with the canonical
    time tau = k*t + i (Sec. 3.2)."""
    k = len(prog.statements)
    for t in range(steps):
        for i, st in enumerate(prog.statements):
            ranges = [range(st.lo[d], N[d] + st.hi[d]) for d in range(prog.dims)]
            for s in product(*ranges):
                yield k * t + i, s, st, t


def dependences(prog: Program, N: Sequence[int], steps: int, typed: bool = False) -> List[Tuple]:
    """All memory-based dependences (RAW, WAR, WAW) between instances, by simulating the
    original execution order over the actual memory locations (Sec. 3.1: 'This dependence
    relation can be computed from the iteration domain, the access relation and a
    description of the original execution order').  Returns pairs
    (source instance, sink instance), instances as (tau, s); with typed=True triples
    (kind, source, sink), kind in {"RAW", "WAR", "WAW"}.

    Memory locations: ping-pong (Fig. 1) -- step t reads A[t%2] and
    writes A[(t+1)%2]; in place (FDTD) -- one copy per array; time-expanded -- step t
    writes A[t] and reads A[t + dt] (no location reused)."""
    last_write: Dict[Tuple, Tuple] = {}
    readers: Dict[Tuple, List[Tuple]] = {}
    deps = []

    def add(kind, src, snk):
        deps.append((kind, src, snk) if typed else (src, snk))

    for tau, s, st, t in instances(prog, N, steps):
        me = (tau, s)
        for i, (arr, o) in enumerate(st.reads):
            loc_s = tuple(s[d] + o[d] for d in range(prog.dims))
            if prog.expanded:
                slot = t + st.versions[i]
            else:
                slot = t % 2 if prog.pingpong else 0
            loc = (arr, slot, loc_s)
            if loc in last_write:
                add("RAW", last_write[loc], me)
            readers.setdefault(loc, []).append(me)
        wslot = t if prog.expanded else ((t + 1) % 2 if prog.pingpong else 0)
        wloc = (st.write, wslot, tuple(s))
        if wloc in last_write:
            add("WAW", last_write[wloc], me)
        for r in readers.get(wloc, []):
            if r != me:
                add("WAR", r, me)
        readers[wloc] = []
        last_write[wloc] = me
    return deps


def typed_distance_vectors(deps) -> Dict[str, set]:
    """{kind: distance vectors} of typed dependences (dependences(..., typed=True))."""
    out: Dict[str, set] = {"RAW": set(), "WAR": set(), "WAW": set()}
    for kind, a, b in deps:
        out[kind].add(tuple([b[0] - a[0]] + [b[1][d] - a[1][d] for d in range(len(a[1]))]))
    return out


def distance_vectors(deps) -> set:
    """Dependence distance vectors (difference in schedule space, Sec. 3.1)."""
    return {tuple([b[0] - a[0]] + [b[1][d] - a[1][d] for d in range(len(a[1]))]) for a, b in deps}


def slopes(distances: Iterable[Tuple[int, int]]) -> Tuple[Fr, Fr]:
    """delta0, delta1 with  ds <= delta0 * dt  and  ds >= -delta1 * dt  for every distance
    (dt, ds) (Sec. 3.3.2, Fig. 3).  The LP optimum is the extreme
    ratio; clamped at 0 so the cone always contains the time axis."""
    d0 = Fr(0)
    d1 = Fr(0)
    for dt, ds in distances:
        assert dt > 0, "the outer dimension must carry every dependence (Sec. 3.3.1)"
        d0 = max(d0, Fr(ds, dt))
        d1 = max(d1, Fr(-ds, dt))
    return d0, d1


def frac(x: Fr) -> Fr:
    """{x} = x - floor(x)."""
    return x - floor(x)


def w0_lower_bound(d0: Fr, d1: Fr, h: int) -> Fr:
    """Eq. (1): w0 >= max(delta0 + {delta0 h}, delta1 + {delta1 h}) - 1."""
    return max(d0 + frac(d0 * h), d1 + frac(d1 * h)) - 1


@dataclass(frozen=True)
class Hex:
    d0: Fr
    d1: Fr
    h: int
    w0: int

    @property
    def F0(self) -> int:
        return floor(self.d0 * self.h)

    @property
    def F1(self) -> int:
        return floor(self.d1 * self.h)

    @property
    def height(self) -> int:  # 2h + 2
        return 2 * self.h + 2

    @property
    def width(self) -> int:  # 2w0 + 2 + floor(d0 h) + floor(d1 h)
        return 2 * self.w0 + 2 + self.F0 + self.F1


def in_hexagon(hx: Hex, a: int, b: int) -> bool:
    """Constraints (6), (7), (8), (10), (12), (13) in the local box coordinates (a, b)
    (PAPER.md:456-538).  d0, d1 are the denominators of delta0, delta1."""
    d0, d1, h, w0 = hx.d0, hx.d1, hx.h, hx.w0
    den0, den1 = d0.denominator, d1.denominator
    c6 = d0 * a - b <= (2 * h + 1) * d0 - hx.F0
    c7 = a <= 2 * h + 1
    c8 = d1 * a + b <= (2 * h + 1) * d1 + hx.F0 + w0
    c10 = d1 * a + b >= h * d1 - Fr(den1 - 1, den1)
    c12 = d0 * a - b >= d0 * h - hx.F0 - w0 - hx.F1 - Fr(den0 - 1, den0)
    c13 = a >= 0
    return c6 and c7 and c8 and c10 and c12 and c13


def box_coords(hx: Hex, t: int, s0: int, phase: int, literal_eq3: bool = False):
    """(T, S0, a, b) of the box of the given phase containing (t, s0): eqs. (2)-(5) and the
    local coordinates of Sec. 3.3.3.  `literal_eq3` uses the extracted
    eq. (3) numerator floor(delta1 h) instead of floor(delta0 h) (reading R1)."""
    H, W = hx.height, hx.width
    c = hx.F1 - hx.F0
    if phase == 0:
        T = (t + hx.h + 1) // H  # eq. (2)
        shift = (hx.F1 if literal_eq3 else hx.F0) + hx.w0 + 1
        n = s0 + shift + T * c  # eq. (3) numerator
        a = (t + hx.h + 1) % H
    else:
        T = t // H  # eq. (4)
        n = s0 + T * c  # eq. (5) numerator
        a = t % H
    return T, n // W, a, n % W


def hex_tile(hx: Hex, t: int, s0: int, literal_eq3: bool = False):
    """(T, p, S0, a, b): the hexagonal tile containing (t, s0), choosing the phase whose box
    contains it inside the hexagon (Sec. 3.6: 'Each phase is only applied to the subset
    of the domain that satisfies (6), (8), (10) and (12)').  Returns a
    list so that tests can detect double or missing coverage."""
    out = []
    for p in (0, 1):
        T, S0, a, b = box_coords(hx, t, s0, p, literal_eq3)
        if in_hexagon(hx, a, b):
            out.append((T, p, S0, a, b))
    return out


def classical(delta1_i: Fr, w_i: int, s_i: int, u: int, trans: int = 0) -> Tuple[int, int]:
    """Eq. (14) S_i = floor((s_i + delta1_i u)/w_i) and eq. (17)
    s'_i = (s_i + delta1_i u) mod w_i, with u the per-phase normalised time of eqs. (15),
    (16); `trans` translates the tiles by a fixed offset ("We allow the
    tiles in the schedule to be translated by manually specifying the translation offset",
    Sec. 4.2.3)."""
    x = s_i - trans + delta1_i * u
    S = floor(x / w_i)
    return S, x - S * w_i


def hybrid(hx: Hex, deltas_i: Sequence[Fr], w: Sequence[int], t: int, s: Sequence[int],
           trans: Sequence[int] = None):
    """[t, s0..sn] -> [T, p, S0..Sn, t', s'0..s'n] (Sec. 3.6).  The
    normalised u of eqs. (15)/(16) equals the local box row a."""
    tiles = hex_tile(hx, t, s[0])
    assert len(tiles) == 1, (t, s, tiles)
    T, p, S0, a, b = tiles[0]
    Ss, sp = [], []
    for i in range(1, len(s)):
        Si, si = classical(deltas_i[i - 1], w[i - 1], s[i], a, trans[i - 1] if trans else 0)
        Ss.append(Si)
        sp.append(si)
    return (T, p, S0, *Ss, a, b, *sp)


def fig6(h: int, w0: int, w: Sequence[int], t: int, s: Sequence[int]):
    """Fig. 6, the paper's printed phase-0 relation for +-1 distances.
    Returns the schedule tuple if (t, s) belongs to phase 0, else None."""
    a = (t + h + 1) % (2 * h + 2)
    b = (s[0] + h + 1 + w0) % (2 * h + 2 + 2 * w0)
    if not (a - b <= h + 1 and a + b <= 3 * h + 1 + w0 and a + b >= h and a - b >= -w0 - h):
        return None
    T = (t + h + 1) // (2 * h + 2)
    S0 = (s[0] + h + 1 + w0) // (2 * h + 2 + 2 * w0)
    Sk = [(s[k] + a) // w[k - 1] for k in range(1, len(s))]
    tp = a
    s0p = b
    skp = [(s[k] + a) % w[k - 1] for k in range(1, len(s))]
    return (T, 0, S0, *Sk, tp, s0p, *skp)


def hexagon_rows(hx: Hex) -> List[Tuple[int, int]]:
    """For each local row a in [0, 2h+1], the inclusive b-range of the hexagon (by
    enumerating the constraints over the box)."""
    rows = []
    for a in range(hx.height):
        bs = [b for b in range(hx.width) if in_hexagon(hx, a, b)]
        rows.append((min(bs), max(bs)) if bs else (1, 0))
    return rows


def check_schedule(prog: Program, N: Sequence[int], steps: int, hx: Hex,
                   deltas_i: Sequence[Fr], w: Sequence[int], literal_eq3: bool = False,
                   trans: Sequence[int] = None):
    """Brute-force validity of the hybrid schedule on a small grid: returns a dict of
    violation counts (all zero for a valid schedule)."""
    sched = {}
    coverage_err = 0
    for tau, s, st, t in instances(prog, N, steps):
        tiles = hex_tile(hx, tau, s[0], literal_eq3)
        if len(tiles) != 1:
            coverage_err += 1
            continue
        T, p, S0, a, b = tiles[0]
        Ss = [classical(deltas_i[i - 1], w[i - 1], s[i], a, trans[i - 1] if trans else 0)[0]
              for i in range(1, len(s))]
        sched[(tau, s)] = ((T, p), S0, tuple(Ss) + (a,))
    order_err = same_phase_err = same_step_err = 0
    for src, snk in dependences(prog, N, steps):
        if src not in sched or snk not in sched:
            continue
        (tp_a, S0a, seq_a), (tp_b, S0b, seq_b) = sched[src], sched[snk]
        if tp_a < tp_b:
            continue
        if tp_a > tp_b:
            order_err += 1
        elif S0a != S0b:
            same_phase_err += 1  # tiles of one (T, p) must be independent
        elif seq_a > seq_b:
            order_err += 1
        elif seq_a == seq_b:
            same_step_err += 1  # points of one (S1..Sn, t') step run in parallel
    return {"coverage": coverage_err, "order": order_err, "same_phase": same_phase_err,
            "same_step": same_step_err, "instances": len(sched)}


def tile_in_out_counts(hx: Hex, radius: int = 1) -> Tuple[int, int, int]:
    """(points, In, Out) of one full hexagon of a 1-D stencil with the given radius along
    s0: points computed, distinct values read from outside the tile, and values produced
    in the tile that are read outside it (or are the top level).  Used to pin the
    closed-form traffic model of DESIGN.md (per classical column)."""
    rows = hexagon_rows(hx)
    pts = {(a, b) for a, (lo, hi) in enumerate(rows) for b in range(lo, hi + 1)}
    ins = set()
    outs = set()
    for a, b in pts:
        for o in range(-radius, radius + 1):
            if (a - 1, b + o) not in pts:
                ins.add((a - 1, b + o))  # value at level a (produced by instance a-1)
            if (a + 1, b - o) not in pts:
                outs.add((a, b))
    return len(pts), len(ins), len(outs)
