"""Multi-process (world_size 2 and 3, gloo backend, CPU) tests of the slab-mode protocol of the
C ABI's distributed plans (csrc/dist.cpp, include/stencil.h stencil_plan_dist).  Each rank takes
its layout and its local plan from the library's host-only stencil_dist_layout /
stencil_dist_local_plan (the exact partition, ghost width and slab launch table -- the global
hexagon tiling translated to the slab -- that stencil_plan_dist runs), then runs the library's
loop (paper_conf_cgo_grosserchsv14_b200.dist.run_protocol: the ghost planes of both ping-pong
buffers exchanged before every launch but the first) with a CPU executor of the launch table
(tests/_schedexec.py) in place of the kernels (there is no GPU here; on the GPU box the launches
are the hybrid kernels and the exchange is NCCL).  The gathered owned planes must be
bit-identical to the single-domain oracle ("bit-identical for every P")."""
import os
import socket
import sys

import numpy as np
import pytest
import torch
import torch.distributed as dist
import torch.multiprocessing as mp

import oracle
import stencil_inputs

sys.path.insert(0, os.path.dirname(os.path.abspath(__file__)))
from paper_conf_cgo_grosserchsv14_b200 import Plan, Stencil
from paper_conf_cgo_grosserchsv14_b200 import dist as hdist


def _free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def _worker(rank, world, port, kind, ext, T, out_dir):
    import _schedexec

    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        plan, lay = hdist.local_plan(kind, ext, T, rank, world, part_dim=int(os.environ.get("HEXS_TEST_PART_DIM", "-1")))
        g = stencil_inputs.uniform(ext, seed=5)
        local = np.ascontiguousarray(lay.take(g, lay.loc_lo, lay.loc_hi))
        assert local.shape == lay.local_ext
        bufs = [torch.from_numpy(local.copy()), torch.from_numpy(local.copy())]
        ex = _schedexec.launch_executor(plan, kind)
        hdist.run_protocol(bufs, lay, plan, lambda ln, b: ex(ln, [x.numpy() for x in b]))
        lo, hi = lay.own_local
        np.save(os.path.join(out_dir, f"r{rank}.npy"), lay.take(bufs[T % 2], lo, hi).numpy())
        np.save(os.path.join(out_dir, f"r{rank}_lo.npy"), np.array([lay.own_lo, lay.part_dim]))
    finally:
        dist.destroy_process_group()


@pytest.mark.parametrize("kind,ext,T,world", [
    ("star2d5", (61, 23), 17, 2),
    ("star2d5", (90, 19), 29, 3),
    ("star3d7", (20, 31, 11), 13, 2),   # 3D default: y (classically tiled) partitioned
    ("star3d7", (23, 44, 10), 11, 3),
])
def test_slab_mode_bit_identical(tmp_path, kind, ext, T, world):
    port = _free_port()
    mp.spawn(_worker, args=(world, port, kind, ext, T, str(tmp_path)), nprocs=world, join=True)
    parts = []
    for r in range(world):
        lo = int(np.load(tmp_path / f"r{r}_lo.npy")[0])
        parts.append((lo, np.load(tmp_path / f"r{r}.npy")))
    pd = int(np.load(tmp_path / "r0_lo.npy")[1])
    parts.sort(key=lambda p: p[0])
    got = np.concatenate([p[1] for p in parts], axis=pd)
    exp = oracle.run(kind, stencil_inputs.uniform(ext, seed=5), T)
    assert got.shape == exp.shape
    assert np.array_equal(got, exp)


@pytest.mark.parametrize("part_dim", [0, 1])
def test_3d_partition_dims(tmp_path, part_dim):
    """3D slabs along the hexagonal dimension (z, tiling translated) and along a classical one (y)."""
    port = _free_port()
    ext, T, world = (26, 28, 9), 10, 2
    os.environ["HEXS_TEST_PART_DIM"] = str(part_dim)
    try:
        mp.spawn(_worker, args=(world, port, "star3d7", ext, T, str(tmp_path)), nprocs=world, join=True)
    finally:
        del os.environ["HEXS_TEST_PART_DIM"]
    parts = sorted((int(np.load(tmp_path / f"r{r}_lo.npy")[0]), np.load(tmp_path / f"r{r}.npy")) for r in range(world))
    got = np.concatenate([p[1] for p in parts], axis=part_dim)
    assert np.array_equal(got, oracle.run("star3d7", stencil_inputs.uniform(ext, seed=5), T))


def test_local_plan_keeps_the_global_tiling():
    """A slab's local plan is the global schedule translated by loc_lo: every instance of the
    slab has the same (T, p, S0, t', s') as in the global plan (Sec. 4.2.3 translation)."""
    ext, T = (61, 23), 17
    gplan = None
    for rank in range(3):
        plan, lay = hdist.local_plan("star2d5", ext, T, rank, 3)
        if gplan is None:  # the global plan with the slabs' hexagon
            gplan = Plan(Stencil("star2d5", ext), T, h=plan.info["h"], w0=plan.info["w0"])
        assert (plan.info["h"], plan.info["w0"], plan.info["W"]) == (gplan.info["h"], gplan.info["w0"], gplan.info["W"])
        for tau in range(0, T, 3):
            for r in range(0, lay.loc_hi - lay.loc_lo, 2):
                for j in range(0, ext[1], 5):
                    loc = plan.schedule_of(tau, (r, j))
                    glob = gplan.schedule_of(tau, (r + lay.loc_lo, j))
                    assert loc[:3] == glob[:3] and loc[4] == glob[4] and loc[5] == glob[5]


def test_layout_properties():
    """The library's partition: owned ranges tile dimension 0 in rank order, ghosts clipped at the
    global boundary, G = radius * D, D a multiple of the hexagon height 2h+2 by default, and the
    ghost share of a 128-index slab of the 1024^3 config stays at or under 12.5%."""
    from paper_conf_cgo_grosserchsv14_b200 import StencilError

    for N0 in (17, 64, 101):
        for P in (1, 2, 3, 4):
            try:
                lays = [hdist.layout("star2d5", (N0, 40), 50, r, P) for r in range(P)]
            except StencilError:  # a slab thinner than the ghost width (one time tile) is refused
                assert P > 1 and N0 // P < 8
                continue
            assert lays[0].own_lo == 0 and lays[-1].own_hi == N0
            for a, b in zip(lays, lays[1:]):
                assert a.own_hi == b.own_lo
            for lay in lays:
                G = lay.ghost
                assert G == lay.time_block == 2 * lay.h + 2  # radius x time-tile depth
                assert lay.loc_lo == max(0, lay.own_lo - G) and lay.loc_hi == min(N0, lay.own_hi + G)
                assert lay.local_ext == (lay.loc_hi - lay.loc_lo, 40)
    for P in (2, 4, 8):
        for r in (0, P // 2, P - 1):
            lay = hdist.layout("star3d7", (1024, 1024, 1024), 256, r, P)
            assert lay.part_dim == 1  # the classically tiled y of the 3D kernels
            assert lay.time_block % (2 * lay.h + 2) == 0
            owned = lay.own_hi - lay.own_lo
            # (3, 7): 2 x 8 ghost lines per 128 owned -- the measured-fastest tile per rank
            assert (lay.loc_hi - lay.loc_lo - owned) / owned <= 0.125, (P, r, lay)
            assert lay.local_ext == (1024, lay.loc_hi - lay.loc_lo, 1024)
    lay = hdist.layout("star3d7", (64, 48, 40), 20, 1, 2, part_dim=0)  # the hexagonal dimension
    assert lay.part_dim == 0 and lay.local_ext[1:] == (48, 40)
    # a slab thinner than the ghost width is refused; FDTD has no slab mode
    with pytest.raises(StencilError):
        hdist.layout("star2d5", (10, 10), 40, 0, 4)
    with pytest.raises(StencilError):
        hdist.layout("fdtd2d", (40, 40), 10, 0, 2)


def test_halo_rows_needed_state():
    """stencil_dist_halo_rows: before every launch each z travels in the buffer of its current
    level, and in the other one exactly where a z-neighbour is one level behind; for the (3, 7)
    hexagon that is ~68 % of both buffers' halo lines (the 1024^3 slabs' exchange volume)."""
    ext, T = (1024, 1024, 1024), 256
    plan, lay = hdist.local_plan("star3d7", ext, T, 3, 8)
    assert lay.part_dim == 1 and (plan.info["h"], plan.info["w0"]) == (3, 7)
    lo, hi = plan.hexagon()
    W = plan.info["W"]
    lev = np.zeros(ext[0], dtype=np.int64)
    total = moved = 0
    for k, ln in enumerate(plan.launches()):
        if k > 0:
            rows = [hdist.halo_rows(plan, 1, k, b) for b in (0, 1)]
            for b in (0, 1):
                exp = [z for z in range(ext[0])
                       if lev[z] % 2 == b or (z > 0 and lev[z - 1] < lev[z]) or (z + 1 < ext[0] and lev[z + 1] < lev[z])]
                assert rows[b] == exp
            assert set(rows[0]) | set(rows[1]) == set(range(ext[0]))
            total += 2 * ext[0]
            moved += len(rows[0]) + len(rows[1])
        for a in range(ln["a_lo"], ln["a_hi"] + 1):
            for S0 in range(ln["S0_lo"], ln["S0_hi"] + 1):
                i0 = S0 * W - ln["row_off"]
                r0, r1 = max(i0 + lo[a], 1), min(i0 + hi[a], ext[0] - 2)
                if r0 <= r1:
                    lev[r0:r1 + 1] = ln["tau0"] + a + 1
            assert np.all(np.abs(np.diff(lev[1:-1])) <= 1)  # adjacent levels differ by <= 1 (ping-pong WAR)
    assert 0.6 < moved / total < 0.75
    # the hexagonal dimension partitioned: every plane travels
    p0, _ = hdist.local_plan("star3d7", (64, 48, 40), 20, 1, 2, part_dim=0)
    assert hdist.halo_rows(p0, 0, 1, 0) is None
