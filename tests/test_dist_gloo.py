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
        plan, lay = hdist.local_plan(kind, ext, T, rank, world)
        g = stencil_inputs.uniform(ext, seed=5)
        local = np.ascontiguousarray(g[lay.loc_lo:lay.loc_hi])
        assert local.shape == lay.local_ext
        bufs = [torch.from_numpy(local.copy()), torch.from_numpy(local.copy())]
        ex = _schedexec.launch_executor(plan, kind)
        hdist.run_protocol(bufs, lay, plan, lambda ln, b: ex(ln, [x.numpy() for x in b]))
        lo, hi = lay.own_local
        np.save(os.path.join(out_dir, f"r{rank}.npy"), bufs[T % 2][lo:hi].numpy())
        np.save(os.path.join(out_dir, f"r{rank}_lo.npy"), np.array([lay.own_lo]))
    finally:
        dist.destroy_process_group()


@pytest.mark.parametrize("kind,ext,T,world", [
    ("star2d5", (61, 23), 17, 2),
    ("star2d5", (90, 19), 29, 3),
    ("star3d7", (40, 9, 11), 13, 2),
    ("star3d7", (44, 8, 10), 11, 3),
])
def test_slab_mode_bit_identical(tmp_path, kind, ext, T, world):
    port = _free_port()
    mp.spawn(_worker, args=(world, port, kind, ext, T, str(tmp_path)), nprocs=world, join=True)
    parts = []
    for r in range(world):
        lo = int(np.load(tmp_path / f"r{r}_lo.npy")[0])
        parts.append((lo, np.load(tmp_path / f"r{r}.npy")))
    parts.sort(key=lambda p: p[0])
    got = np.concatenate([p[1] for p in parts], axis=0)
    exp = oracle.run(kind, stencil_inputs.uniform(ext, seed=5), T)
    assert got.shape == exp.shape
    assert np.array_equal(got, exp)


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
    ghost share of a 128-plane slab of the 1024^3 config stays under 12%."""
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
            assert lay.time_block % (2 * lay.h + 2) == 0
            owned = lay.own_hi - lay.own_lo
            assert (lay.loc_hi - lay.loc_lo - owned) / owned <= 0.12, (P, r, lay)
    # a slab thinner than the ghost width is refused; FDTD has no slab mode
    with pytest.raises(StencilError):
        hdist.layout("star2d5", (10, 10), 40, 0, 4)
    with pytest.raises(StencilError):
        hdist.layout("fdtd2d", (40, 40), 10, 0, 2)
