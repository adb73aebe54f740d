"""The Table 4 replay executors (include/stencil.h STENCIL_EXEC_T4A..T4F, kernels/ablation.cu):
the optimisation ablation of Sec. 6.2 as six memory strategies of one 3D
hybrid phase kernel.  Host tests check the plan (Table 4's tile and CTA shape, the alignment
translation of (d)-(f)); GPU tests hold every configuration to the oracle bit for bit."""
import numpy as np
import pytest

import oracle
import stencil_inputs
from paper_conf_cgo_grosserchsv14_b200 import Plan, Stencil, StencilError

CFGS = ["t4a", "t4b", "t4c", "t4d", "t4e", "t4f"]


@pytest.mark.parametrize("cfg", CFGS)
def test_plan_uses_table4_setup(cfg):
    """h = 2, w0 = 7, w1 = 10, w2 = 32; the executor and kernel reported."""
    plan = Plan(Stencil("box3d27", (64, 70, 96)), 12, executor=cfg)
    info = plan.info
    assert (info["h"], info["w0"], info["w"][0], info["w"][1]) == (2, 7, 10, 32)
    assert info["executor"] == 3 + CFGS.index(cfg) and plan.executor_name == "ablation"
    assert info["delta_cls"][:2] == [1, 1]


def test_alignment_translation():
    """(d) puts the copy-in box start B2 - H on a 128-B line, (e)/(f) the 32 columns every later
    x tile loads ([B2 + 1, B2 + 33)); (a)-(c) keep the untranslated tiling."""
    st = Stencil("star3d7", (40, 40, 256))
    H = 6
    for cfg, want in [("t4a", 0), ("t4b", 0), ("t4c", 0), ("t4d", H % 32), ("t4e", 31), ("t4f", 31)]:
        ct = Plan(st, 8, executor=cfg).info["trans_cls"][1]
        assert ct == want
        if cfg == "t4d":
            assert (32 * 5 + ct - H) % 32 == 0  # box start of any full-launch x tile
        if cfg in ("t4e", "t4f"):
            assert (32 * 5 + ct + 1) % 32 == 0


def test_schedule_unchanged_by_translation():
    """The translation moves the classical tile boundaries only: every instance keeps its
    hexagon coordinates (T, p, S0, t') and the whole launch table covers the same levels."""
    st = Stencil("star3d7", (30, 26, 70))
    a, d = Plan(st, 9, executor="t4a"), Plan(st, 9, executor="t4d")
    for tau in range(0, 9):
        for s in [(5, 7, 9), (17, 3, 64), (28, 20, 1)]:
            sa, sd = a.schedule_of(tau, s), d.schedule_of(tau, s)
            assert sa[:3] == sd[:3]
    assert [(l["T"], l["phase"]) for l in a.launches()] == [(l["T"], l["phase"]) for l in d.launches()]


@pytest.mark.parametrize("kind,dtype,tile", [("star2d5", "float32", {}), ("jacobi2d5", "float32", {}),
                                             ("box3d27", "float64", {}), ("star3d7", "float32",
                                                                          {"w": (8, 32, 0)})])
def test_unsupported_setups_refused(kind, dtype, tile):
    ext = (32, 40) if kind.endswith("2d5") else (20, 20, 64)
    with pytest.raises(StencilError):
        Plan(Stencil(kind, ext, dtype=dtype), 6, executor="t4c", **tile)


# ---- GPU parity ---------------------------------------------------------------------

CASES = [("box3d27", (38, 45, 70), 11, 1), ("star3d7", (64, 40, 96), 13, 2), ("gradient3d", (29, 33, 130), 7, 3),
         ("box3d27", (70, 23, 33), 6, 4), ("star3d7", (5, 70, 200), 17, 5)]


@pytest.mark.gpu
@pytest.mark.parametrize("cfg", CFGS)
@pytest.mark.parametrize("case", range(len(CASES)))
def test_ablation_parity(cfg, case):
    torch = pytest.importorskip("torch")
    kind, shape, T, seed = CASES[case]
    g = stencil_inputs.uniform(shape, seed=seed, dtype=np.float32)
    plan = Plan(Stencil(kind, shape), T, executor=cfg)
    out = plan.run(torch.from_numpy(g).cuda())
    torch.cuda.synchronize()
    got = out.cpu().numpy()
    exp = oracle.run(kind, g, T)
    if not np.array_equal(got, exp):
        bad = np.argwhere(got != exp)
        raise AssertionError(f"{cfg} {kind} {shape}: {len(bad)} mismatches, first {tuple(bad[0])}")


@pytest.mark.gpu
@pytest.mark.parametrize("h,w0", [(1, 3), (3, 4)])
def test_ablation_other_tiles(h, w0):
    torch = pytest.importorskip("torch")
    shape, T = (41, 37, 100), 15
    g = stencil_inputs.uniform(shape, seed=9, dtype=np.float32)
    exp = oracle.run("box3d27", g, T)
    for cfg in CFGS:
        plan = Plan(Stencil("box3d27", shape), T, h=h, w0=w0, executor=cfg)
        got = plan.run(torch.from_numpy(g).cuda()).cpu().numpy()
        assert np.array_equal(got, exp), (cfg, h, w0)
