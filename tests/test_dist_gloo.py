"""Multi-process (world_size 2 and 3, gloo backend, CPU) tests of the slab-partition / halo
exchange / time-block logic of paper_conf_cgo_grosserchsv14_b200.dist.  The per-block
compute is injected (the oracle's naive loop) because there is no GPU here; on the GPU box
the same SlabRunner calls the C-ABI hybrid kernels.  The gathered result must be
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


def _worker(rank, world, port, kind, ext, T, D, out_dir):
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        def compute(local, steps):  # test-only injection of the CPU oracle
            local.copy_(torch.from_numpy(oracle.run(kind, local.numpy(), steps)))

        runner = hdist.SlabRunner(kind, ext, T, D=D, compute=compute)
        g = stencil_inputs.uniform(ext, seed=5)
        local = torch.from_numpy(np.ascontiguousarray(runner.scatter_view(g)))
        runner.run(local)
        lo, hi = runner.slab.own_local
        np.save(os.path.join(out_dir, f"r{rank}.npy"), local[lo:hi].numpy())
        np.save(os.path.join(out_dir, f"r{rank}_lo.npy"), np.array([runner.slab.own_lo]))
    finally:
        dist.destroy_process_group()


@pytest.mark.parametrize("kind,ext,T,D,world", [
    ("star2d5", (41, 23), 17, 4, 2),
    ("box2d9", (50, 19), 13, 5, 3),
    ("jacobi2d5", (30, 30), 9, 9, 2),
    ("star3d7", (22, 9, 11), 7, 3, 2),
])
def test_slab_mode_bit_identical(tmp_path, kind, ext, T, D, world):
    port = _free_port()
    mp.spawn(_worker, args=(world, port, kind, ext, T, D, str(tmp_path)), nprocs=world, join=True)
    parts = []
    for r in range(world):
        lo = int(np.load(tmp_path / f"r{r}_lo.npy")[0])
        parts.append((lo, np.load(tmp_path / f"r{r}.npy")))
    parts.sort(key=lambda p: p[0])
    got = np.concatenate([p[1] for p in parts], axis=0)
    exp = oracle.run(kind, stencil_inputs.uniform(ext, seed=5), T)
    assert got.shape == exp.shape
    assert np.array_equal(got, exp)


def test_partition_properties():
    for N0 in (17, 64, 101):
        for P in (1, 2, 3, 4):
            for G in (1, 2, 3):
                slabs = [hdist.partition(N0, P, r, G) for r in range(P)]
                assert slabs[0].own_lo == 0 and slabs[-1].own_hi == N0
                for a, b in zip(slabs, slabs[1:]):
                    assert a.own_hi == b.own_lo
                for s in slabs:
                    assert s.loc_lo == max(0, s.own_lo - G) and s.loc_hi == min(N0, s.own_hi + G)
    with pytest.raises(ValueError):
        hdist.partition(10, 4, 0, 5)
    assert hdist.time_blocks(17, 4) == [4, 4, 4, 4, 1]
    assert hdist.time_blocks(8, 8) == [8]
