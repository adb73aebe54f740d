"""Multi-process (world_size 2 and 3, gloo backend, CPU) tests of the slab-mode protocol of the
C ABI's distributed plans (csrc/dist.cpp, include/stencil.h stencil_plan_dist).  Each rank takes
its layout from the library's host-only stencil_dist_layout (the exact partition, ghost width and
time block stencil_plan_dist uses), runs the library's block loop (paper_conf_cgo_grosserchsv14_b200
.dist.run_protocol: halo exchange between blocks, D steps per block on the local slab) with the
CPU oracle injected as the per-block compute (there is no GPU here; on the GPU box the blocks run
the hybrid kernels and the exchange is NCCL), and the gathered owned planes must be
bit-identical to the single-domain oracle ("bit-identical for every P")."""
import os
import socket

import numpy as np
import pytest
import torch
import torch.distributed as dist
import torch.multiprocessing as mp

import oracle
import stencil_inputs
from paper_conf_cgo_grosserchsv14_b200 import dist as hdist


def _free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def _worker(rank, world, port, kind, ext, T, block, out_dir):
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    if block:
        os.environ["HEXS_TIME_BLOCK"] = str(block)
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        lay = hdist.layout(kind, ext, T, rank, world)

        def compute(local, steps):  # test-only injection of the CPU oracle (the local slab alone)
            local.copy_(torch.from_numpy(oracle.run(kind, local.numpy(), steps)))

        g = stencil_inputs.uniform(ext, seed=5)
        local = torch.from_numpy(np.ascontiguousarray(g[lay.loc_lo:lay.loc_hi]))
        assert tuple(local.shape) == lay.local_ext
        hdist.run_protocol(local, lay, T, compute)
        lo, hi = lay.own_local
        np.save(os.path.join(out_dir, f"r{rank}.npy"), local[lo:hi].numpy())
        np.save(os.path.join(out_dir, f"r{rank}_lo.npy"), np.array([lay.own_lo]))
    finally:
        dist.destroy_process_group()


@pytest.mark.parametrize("kind,ext,T,block,world", [
    ("star2d5", (41, 23), 17, 4, 2),
    ("box2d9", (50, 19), 13, 5, 3),
    ("jacobi2d5", (30, 30), 9, 0, 2),
    ("star3d7", (22, 9, 11), 7, 3, 2),
    ("star3d7", (40, 9, 12), 13, 0, 3),
    ("gradient3d", (26, 8, 8), 8, 0, 2),
])
def test_slab_mode_bit_identical(tmp_path, kind, ext, T, block, world):
    port = _free_port()
    mp.spawn(_worker, args=(world, port, kind, ext, T, block, str(tmp_path)), nprocs=world, join=True)
    parts = []
    for r in range(world):
        lo = int(np.load(tmp_path / f"r{r}_lo.npy")[0])
        parts.append((lo, np.load(tmp_path / f"r{r}.npy")))
    parts.sort(key=lambda p: p[0])
    got = np.concatenate([p[1] for p in parts], axis=0)
    exp = oracle.run(kind, stencil_inputs.uniform(ext, seed=5), T)
    assert got.shape == exp.shape
    assert np.array_equal(got, exp)


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
                assert G == lay.time_block
                assert lay.loc_lo == max(0, lay.own_lo - G) and lay.loc_hi == min(N0, lay.own_hi + G)
                assert lay.local_ext == (lay.loc_hi - lay.loc_lo, 40)
                assert sum(lay.blocks(50)) == 50 and len(lay.blocks(50)) == lay.n_blocks
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
