"""Chained 3D launches (csrc/kernels/hex3d.cu wait_prev, DESIGN.md §6.2 "chained launches"): before
a tile's first fill its producer acquires the flags of every tile of launches k-1 and k-2 whose
write box meets the tile's read box.  Checked here by brute force on the planner's schedule: for
every stencil instance, the instance that wrote each value it reads lies (i) in the same launch and
an earlier-or-equal classical tile (the in-launch wavefront), or (ii) in launch k-1 or k-2 and
inside the ranges the kernel's formula gives -- never in any other launch."""
import numpy as np
import pytest

from paper_conf_cgo_grosserchsv14_b200 import Plan, Stencil

SIGMA = 4  # x skew per level of the 3D kernel


def fdiv(a, b):
    return a // b  # Python floors


def cdiv(a, b):
    return -((-a) // b)


def writer_ranges(reader, writer, W, Q, NY, NX, S0r, S1r, S2r):
    """The kernel's writer-tile ranges (hex3d.cu wait_prev), restated from DESIGN.md §6.2."""
    D = reader["tau0"] - writer["tau0"] - 1
    i0 = S0r * W - reader["row_off"]
    zlo, zhi = i0 - 1, i0 + Q - 2
    s0 = (cdiv(zlo - (Q - 3) + writer["row_off"], W), fdiv(zhi + writer["row_off"], W))
    s1 = (cdiv(S1r * NY - NY + D, NY), fdiv(S1r * NY + NY + D, NY))
    s2 = (cdiv(S2r * NX - NX + SIGMA * D, NX), fdiv(S2r * NX + NX + SIGMA * D, NX))
    return s0, s1, s2


@pytest.mark.parametrize("h,w0,NY,NX,shape,T", [(3, 7, 32, 32, (40, 90, 100), 20), (2, 7, 16, 32, (30, 50, 70), 14),
                                                 (1, 3, 16, 32, (22, 40, 60), 11)])
def test_chained_launch_dependences_are_covered(h, w0, NY, NX, shape, T):
    plan = Plan(Stencil("star3d7", shape), T, h=h, w0=w0, executor="generic")
    L = plan.launches()
    idx = {(l["T"], l["phase"]): k for k, l in enumerate(L)}
    W = 2 * w0 + 2 + 2 * h
    Q = w0 + 2 * h + 3
    Z, Y, X = shape
    # hexagon of every (tau, z) instance: launch index and S0 (y / x do not enter the hexagon)
    lk = np.full((T, Z), -1, np.int64)
    s0 = np.zeros((T, Z), np.int64)
    for tau in range(T):
        for z in range(1, Z - 1):
            o = plan.schedule_of(tau, (z, 1, 1))
            lk[tau, z] = idx[(o[0], o[1])]
            s0[tau, z] = o[2]
    ys = np.arange(Y)[:, None]
    xs = np.arange(X)[None, :]
    checked = 0
    for tau in range(1, T):
        for z in range(1, Z - 1):
            kr = lk[tau, z]
            lr = L[kr]
            ar = tau - lr["tau0"]
            S1r = fdiv(ys + ar, NY)  # reader tiles of every (y, x)
            S2r = fdiv(xs + SIGMA * ar, NX)
            for dz, dy, dx in ((0, 0, 0), (-1, 0, 0), (1, 0, 0), (0, -1, 0), (0, 1, 0), (0, 0, -1), (0, 0, 1)):
                zw = z + dz
                if zw < 1 or zw > Z - 2:
                    continue  # a boundary value: never written
                kw = lk[tau - 1, zw]
                lw = L[kw]
                aw = tau - 1 - lw["tau0"]
                yw = np.clip(ys + dy, 1, Y - 2)
                xw = np.clip(xs + dx, 1, X - 2)
                S1w = fdiv(yw + aw, NY) + 0 * xw
                S2w = fdiv(xw + SIGMA * aw, NX) + 0 * yw
                inner = (ys >= 1) & (ys <= Y - 2) & (xs >= 1) & (xs <= X - 2)
                if kw == kr:  # in-launch: an earlier-or-equal tile of the same hexagon
                    assert s0[tau - 1, zw] == s0[tau, z]
                    assert np.all(((S1w <= S1r) & (S2w <= S2r))[inner])
                    continue
                assert kr - kw in (1, 2), (kr, kw)  # only the previous two launches
                # per reader tile: the writer's tile inside the formula's ranges
                S1rb = np.broadcast_to(S1r, (Y, X))
                S2rb = np.broadcast_to(S2r, (Y, X))
                for s1r in np.unique(S1rb[inner]):
                    for s2r in np.unique(S2rb[inner][S1rb[inner] == s1r]):
                        m = inner & (S1rb == s1r) & (S2rb == s2r)
                        r0, r1, r2 = writer_ranges(lr, lw, W, Q, NY, NX, int(s0[tau, z]), int(s1r), int(s2r))
                        assert r0[0] <= s0[tau - 1, zw] <= r0[1]
                        assert np.all((S1w[m] >= r1[0]) & (S1w[m] <= r1[1]))
                        assert np.all((S2w[m] >= r2[0]) & (S2w[m] <= r2[1]))
                        checked += int(m.sum())
    assert checked > 0
