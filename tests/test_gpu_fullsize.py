"""Full-grid GPU parity at the BASELINE.json config sizes, in the launch configuration
bench.py times (auto tile, fast kernels, CUDA-graph replay from the second run), plus fp64 at
sizes spanning many tiles.  Every element is compared with the CPU oracle (OpenMP over the
outer dimension; points within a step are independent, so the oracle is bit-identical at any
thread count).  The bar is bit-exact equality (north star: FMA contraction off, identical
per-point expression order)."""
import numpy as np
import pytest

import oracle
import stencil_inputs

torch = pytest.importorskip("torch")
pytestmark = [pytest.mark.gpu, pytest.mark.slow]

from paper_conf_cgo_grosserchsv14_b200 import Plan, Stencil  # noqa: E402


def _nthreads():
    return oracle.max_threads()


def assert_bitexact(got, exp, what=""):
    if not np.array_equal(got, exp):
        diff = np.argwhere(got != exp)
        i = tuple(diff[0])
        raise AssertionError(f"{what}: {len(diff)} mismatches, first at {i}: got {got[i]!r} want {exp[i]!r}")


def _bench_like_run(kind, g, T, runs=3, **tile):
    """Plan once, run `runs` times on the same buffers (eager, capture, graph replay), return
    the last result and the plan."""
    st = Stencil(kind, g.shape, dtype=g.dtype)
    plan = Plan(st, T, **tile)
    x = torch.from_numpy(g).cuda()
    out = torch.empty_like(x)
    for _ in range(runs):
        out.fill_(-1)
        plan.run(x, out)
    torch.cuda.synchronize()
    res = out.cpu().numpy()
    del x, out
    torch.cuda.empty_cache()
    return res, plan


@pytest.mark.parametrize("kind", ["star2d5", "box2d9", "gradient2d"])
def test_2d_config_full_grid(kind):
    """configs[1] (heat-2D 5-/9-point 8192^2, T=512) and gradient-2D at the same size: the whole
    grid, including the aligned multi-chunk default kernel of every class."""
    N, T = 8192, 512
    g = stencil_inputs.uniform((N, N), seed=0)
    got, plan = _bench_like_run(kind, g, T)
    assert plan.info["fast_kernel"] == 1
    exp = oracle.run(kind, g, T, nthreads=_nthreads())
    assert_bitexact(got, exp, f"{kind} 8192^2 T=512")


@pytest.mark.parametrize("kind", ["star3d7", "gradient3d", "box3d27"])
def test_3d_config_full_grid(kind):
    """configs[3] (heat-3D 7-point and gradient-3D 512^3, T=128) and the paper's 27-point heat
    3D at the same size: the whole grid."""
    N, T = 512, 128
    g = stencil_inputs.uniform((N, N, N), seed=0)
    got, plan = _bench_like_run(kind, g, T)
    assert plan.info["fast_kernel"] == 1
    exp = oracle.run(kind, g, T, nthreads=_nthreads())
    assert_bitexact(got, exp, f"{kind} 512^3 T=128")


def test_heat3d_1024_full_grid():
    """configs[4] at N = 1 (heat-3D 7-point 1024^3, T=256): the whole 4 GiB grid."""
    N, T = 1024, 256
    g = stencil_inputs.uniform((N, N, N), seed=0)
    got, plan = _bench_like_run("star3d7", g, T, runs=2)
    assert plan.info["fast_kernel"] == 1
    exp = oracle.run("star3d7", g, T, nthreads=_nthreads())
    del g
    assert_bitexact(got, exp, "star3d7 1024^3 T=256")


@pytest.mark.parametrize("kind,shape,T", [
    ("star2d5", (1024, 1536), 64), ("box2d9", (1030, 1100), 40), ("gradient2d", (1024, 1024), 33),
    ("jacobi2d5", (2048, 1024), 50),
    ("star3d7", (128, 128, 128), 32), ("gradient3d", (130, 140, 128), 21), ("box3d27", (128, 132, 136), 18),
])
def test_fp64_large(kind, shape, T):
    """fp64 on grids of >= 1024^2 / 128^3 (many hexagons, chunks and classical tiles)."""
    g = stencil_inputs.uniform(shape, seed=4, dtype=np.float64)
    got, plan = _bench_like_run(kind, g, T)
    exp = oracle.run(kind, g, T, nthreads=_nthreads())
    assert_bitexact(got, exp, f"{kind} fp64 {shape} T={T}")
