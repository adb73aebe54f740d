"""GPU parity: the CUDA path (through the C ABI) against the CPU oracle, element by element
on the same seeded inputs.  Built with --fmad=false and IEEE div/sqrt, the kernels evaluate
the oracle's expression tree exactly, so the bar is bit-exact equality for every class and
both precisions (BASELINE.json north star: "bit-exactly when both are built with FMA
contraction off and the same per-point expression order")."""
import numpy as np
import pytest

import oracle
import stencil_inputs

torch = pytest.importorskip("torch")
pytestmark = pytest.mark.gpu

from paper_conf_cgo_grosserchsv14_b200 import Plan, Stencil  # noqa: E402


def _gpu_run(kind, grid, T, dtype, **tile):
    st = Stencil(kind, grid.shape, dtype=dtype)
    plan = Plan(st, T, **tile)
    x = torch.from_numpy(grid).cuda()
    out = plan.run(x)
    torch.cuda.synchronize()
    return out.cpu().numpy(), plan


def _gpu_fdtd(fields, T, dtype, **tile):
    st = Stencil("fdtd2d", fields[0].shape, dtype=dtype)
    plan = Plan(st, T, **tile)
    xs = [torch.from_numpy(f).cuda() for f in fields]
    outs = plan.run(xs)
    torch.cuda.synchronize()
    return [o.cpu().numpy() for o in outs], plan


def assert_bitexact(got, exp, what=""):
    if not np.array_equal(got, exp):
        diff = np.argwhere(got != exp)
        i = tuple(diff[0])
        raise AssertionError(f"{what}: {len(diff)} mismatches, first at {i}: got {got[i]!r} want {exp[i]!r}")


KIND2D = ["jacobi2d5", "star2d5", "box2d9", "gradient2d"]
KIND3D = ["star3d7", "gradient3d", "box3d27"]


@pytest.mark.parametrize("kind", KIND2D)
@pytest.mark.parametrize("dtype", [np.float32, np.float64])
@pytest.mark.parametrize("executor", ["auto", "generic", "naive"])
def test_2d_small_ragged(kind, dtype, executor):
    """256x256 T=32 (configs[0]) and a ragged 131x1037 grid, T not a multiple of 2h+2."""
    for shape, T, seed in [((256, 256), 32, 1), ((131, 1037), 13, 2)]:
        g = stencil_inputs.uniform(shape, seed=seed, dtype=dtype)
        got, plan = _gpu_run(kind, g, T, dtype, executor=executor)
        assert_bitexact(got, oracle.run(kind, g, T), f"{kind} {dtype.__name__} {executor} {shape}")


@pytest.mark.parametrize("h,w0", [(3, 7), (1, 3), (3, 10), (2, 5), (4, 5)])
def test_fast2d_tiles_multi_chunk(h, w0):
    """Every compiled star2d5 tile on grids spanning several super-chunks, aligned and
    unaligned rows, with hexagons cut by the domain and by t = 0 / t = T."""
    for shape, T in [((300, 2052), 23), ((97, 1601), 11), ((64, 515), 2 * h + 2)]:
        g = stencil_inputs.uniform(shape, seed=3)
        got, plan = _gpu_run("star2d5", g, T, np.float32, h=h, w0=w0)
        assert plan.info["fast_kernel"] == 1
        assert_bitexact(got, oracle.run("star2d5", g, T), f"h={h} w0={w0} {shape} T={T}")


@pytest.mark.parametrize("kind", ["jacobi2d5", "box2d9"])
def test_fast2d_other_tiles(kind):
    h, w0 = (1, 3) if kind == "jacobi2d5" else (3, 5)
    g = stencil_inputs.uniform((200, 1300), seed=6)
    got, plan = _gpu_run(kind, g, 17, np.float32, h=h, w0=w0)
    assert plan.info["fast_kernel"] == 1
    assert_bitexact(got, oracle.run(kind, g, 17), kind)


def test_2d_edge_cases():
    g = stencil_inputs.uniform((37, 41), seed=8)
    for T in (0, 1, 2, 7, 8, 9):
        got, _ = _gpu_run("star2d5", g, T, np.float32)
        assert_bitexact(got, oracle.run("star2d5", g, T), f"T={T}")
    # minimal grid and a single interior row / column
    for shape in [(3, 3), (3, 700), (700, 3), (4, 5)]:
        g = stencil_inputs.uniform(shape, seed=9)
        got, _ = _gpu_run("box2d9", g, 10, np.float32)
        assert_bitexact(got, oracle.run("box2d9", g, 10), f"{shape}")


def test_in_place_alias():
    g = stencil_inputs.uniform((150, 600), seed=10)
    st = Stencil("star2d5", g.shape)
    plan = Plan(st, 21)
    x = torch.from_numpy(g).cuda()
    plan.run(x, out=x)
    torch.cuda.synchronize()
    assert_bitexact(x.cpu().numpy(), oracle.run("star2d5", g, 21), "in place")


@pytest.mark.parametrize("dtype", [np.float32, np.float64])
@pytest.mark.parametrize("executor", ["auto", "generic", "naive"])
def test_fdtd(dtype, executor):
    for shape, T in [((64, 80), 9), ((101, 257), 17)]:
        f = stencil_inputs.fields(shape, seed=20, n=3, dtype=dtype)
        got, _ = _gpu_fdtd(f, T, dtype, executor=executor)
        exp = oracle.fdtd(*f, T)
        for name, a, b in zip(("ex", "ey", "hz"), got, exp):
            assert_bitexact(a, b, f"fdtd {name} {executor} {shape}")


@pytest.mark.parametrize("dtype", [np.float32, np.float64])
@pytest.mark.parametrize("shape,T,h,w0", [((64, 80), 9, 0, 0), ((101, 260), 17, 0, 0), ((37, 132), 13, 2, 0),
                                          ((90, 72), 11, 5, 3), ((70, 200), 25, 3, 1), ((130, 68), 8, 8, 4),
                                          ((9, 4), 5, 0, 0), ((300, 324), 30, 5, 5),
                                          # the compile-time unrolled (11, 5) kernel: several
                                          # hexagons, both row edges, ragged chunks, full and cut launches
                                          ((200, 332), 40, 11, 5), ((57, 1000), 19, 11, 5)])
def test_fdtd_fast_kernel(dtype, shape, T, h, w0):
    """The shared-memory-ring FDTD kernel (kernels/fdtd.cu): ragged chunk tails, hexagons cut
    by the grid, partial first/last launches, tiny grids -- bit-exact against the oracle."""
    f = stencil_inputs.fields(shape, seed=22, n=3, dtype=dtype)
    got, plan = _gpu_fdtd(f, T, dtype, h=h, w0=w0)
    assert plan.info["fast_kernel"] == 1
    exp = oracle.fdtd(*f, T)
    for name, a, b in zip(("ex", "ey", "hz"), got, exp):
        assert_bitexact(a, b, f"fdtd fast {name} {shape} h={h} w0={w0}")


@pytest.mark.parametrize("h,w0", [(2, 0), (5, 3), (3, 1)])
def test_fdtd_tiles(h, w0):
    f = stencil_inputs.fields((90, 70), seed=21, n=3)
    got, _ = _gpu_fdtd(f, 11, np.float32, h=h, w0=w0)
    exp = oracle.fdtd(*f, 11)
    for a, b in zip(got, exp):
        assert_bitexact(a, b, f"fdtd h={h} w0={w0}")


@pytest.mark.parametrize("kind", KIND3D)
@pytest.mark.parametrize("dtype", [np.float32, np.float64])
@pytest.mark.parametrize("executor", ["auto", "generic", "naive"])
def test_3d(kind, dtype, executor):
    # unaligned rows run the generic wavefront; rows with 16-B aligned strides the TMA kernel
    for shape, T in [((34, 29, 67), 7), ((20, 40, 33), 12), ((30, 37, 68), 9), ((23, 51, 100), 13)]:
        g = stencil_inputs.uniform(shape, seed=30, dtype=dtype)
        got, plan = _gpu_run(kind, g, T, dtype, executor=executor)
        if executor == "auto" and shape[2] % 4 == 0:
            assert plan.info["fast_kernel"] == 1
        assert_bitexact(got, oracle.run(kind, g, T), f"{kind} {executor} {shape}")


@pytest.mark.parametrize("h,w0", [(2, 7), (1, 3), (3, 2)])
def test_fast3d_tiles(h, w0):
    """The tile-wavefront 3D kernel (hexagons over (t, z), hex_dim = 0)."""
    g = stencil_inputs.uniform((41, 70, 96), seed=31)
    got, plan = _gpu_run("star3d7", g, 11, np.float32, h=h, w0=w0, hex_dim=0)
    assert plan.executor_name == "fast3d"
    assert_bitexact(got, oracle.run("star3d7", g, 11), f"fast3d h={h} w0={w0}")


# (requested w[0] -- 0: the variant table's default --, expected (y, x) tile)
@pytest.mark.parametrize("kind,h,w0,wy,tile_yx", [("star3d7", 3, 7, 0, (16, 64)), ("star3d7", 3, 7, 32, (32, 32)),
                                                ("star3d7", 3, 7, 8, (8, 128)), ("star3d7", 2, 7, 16, (16, 32)),
                                                ("box3d27", 2, 7, 16, (16, 64)), ("gradient3d", 2, 7, 16, (16, 64)),
                                                ("box3d27", 2, 7, 0, (32, 32))])
@pytest.mark.parametrize("shape,T", [((70, 150, 140), 13), ((40, 90, 300), 9), ((19, 33, 68), 20)])
def test_fast3d_tile_shapes(kind, h, w0, wy, tile_yx, shape, T):
    """The 3D tile-wavefront variants of every (y, x) tile shape -- the default 16 x 64 of star3d7
    (3, 7), 32 x 32, 8 x 128 (one line per warp), 16 x 32, and the 27-point / gradient 16 x 64 --
    on grids spanning several tiles with ragged edges, hexagons cut at t = 0 / t = T."""
    g = stencil_inputs.uniform(shape, seed=33)
    tile = {"h": h, "w0": w0, "hex_dim": 0}
    if wy:
        tile["w"] = [wy, 0, 0]
    got, plan = _gpu_run(kind, g, T, np.float32, **tile)
    assert plan.executor_name == "fast3d" and tuple(plan.info["w"][:2]) == tile_yx
    assert_bitexact(got, oracle.run(kind, g, T), f"fast3d {kind} ({h},{w0}) {tile_yx} {shape} T={T}")


@pytest.mark.parametrize("kind,h,w0", [("star3d7", 2, 7), ("star3d7", 1, 3), ("star3d7", 3, 5), ("star3d7", 1, 7),
                                       ("star3d7", 2, 5), ("star3d7", 3, 7), ("gradient3d", 2, 7),
                                       ("gradient3d", 1, 7)])
@pytest.mark.parametrize("shape,T", [((41, 70, 96), 11), ((20, 33, 200), 17), ((9, 100, 64), 6), ((33, 5, 132), 9),
                                     ((3, 40, 68), 5), ((50, 47, 4), 8)])
def test_stream3d_tiles(kind, h, w0, shape, T):
    """The streaming 3D kernel (hexagons over (t, y), z streamed, x strips): several strips,
    hexagons cut by the grid and by t = 0 / t = T, degenerate extents (3 planes, 5 rows,
    4 columns), T not a multiple of 2h+2."""
    g = stencil_inputs.uniform(shape, seed=32)
    got, plan = _gpu_run(kind, g, T, np.float32, h=h, w0=w0, hex_dim=1)
    assert plan.executor_name == "stream3d" and plan.info["hex_dim"] == 1
    assert_bitexact(got, oracle.run(kind, g, T), f"stream3d {kind} h={h} w0={w0} {shape} T={T}")


def test_constant_field_full_size_property():
    """Any size: a constant field 1.0 is a fixpoint of star2d5 (coefficients sum to 1)."""
    g = np.ones((8192, 8192), np.float32)
    got, _ = _gpu_run("star2d5", g, 16, np.float32)
    assert np.all(got == 1)


@pytest.mark.slow
def test_full_size_fdtd():
    """configs[2] (fdtd-2D 8192^2, T=500) in the bench's launch configuration, whole fields."""
    f = stencil_inputs.fields((8192, 8192), seed=0, n=3)
    got, plan = _gpu_fdtd(f, 500, np.float32)
    assert plan.info["fast_kernel"] == 1
    exp = oracle.fdtd(*[x.copy() for x in f], 500, nthreads=oracle.max_threads())
    for a, b, name in zip(got, exp, ("ex", "ey", "hz")):
        assert_bitexact(a, b, f"fdtd 8192^2 T=500 {name}")


def test_dist_plan_nccl_single_rank():
    """The C ABI's distributed plan (stencil_plan_dist: NCCL communicator from a unique id, the
    local plan on the slab) with one rank on the GPU: bit-exact against the single-domain oracle
    for 2D and 3D classes and both partition dimensions of a 3D grid."""
    from paper_conf_cgo_grosserchsv14_b200 import dist as hdist

    for kind, ext, T, pd in [("star2d5", (301, 517), 37, -1), ("star3d7", (40, 45, 68), 11, -1),
                             ("star3d7", (64, 40, 64), 20, 0), ("box2d9", (130, 260), 19, -1),
                             ("star3d7", (33, 70, 132), 17, 1)]:
        g = stencil_inputs.uniform(ext, seed=9)
        dp = hdist.DistPlan(kind, ext, T, part_dim=pd)
        lay = dp.layout
        assert lay.part_dim == (pd if pd >= 0 else (1 if len(ext) == 3 else 0))
        assert lay.loc_lo == 0 and lay.loc_hi == ext[lay.part_dim] and lay.local_ext == ext
        local = dp.scatter(g)
        out = torch.empty_like(local)
        for _ in range(2):
            dp.run(local, out)
        torch.cuda.synchronize()
        assert_bitexact(dp.owned(out).cpu().numpy(), oracle.run(kind, g, T), f"dist {kind} part_dim={pd}")

@pytest.mark.parametrize("kind,shape,T", [("star2d5", (300, 1030), 19), ("box2d9", (257, 1100), 12),
                                          ("star3d7", (40, 45, 68), 11), ("box3d27", (30, 37, 68), 9)])
def test_graph_replay_pointer_sets(kind, shape, T):
    """A plan run many times (eager, capture, graph replays) with two pointer sets, in place
    and out of place: every run equals the oracle (the CUDA-graph path of stencil_run)."""
    g = stencil_inputs.uniform(shape, seed=12)
    exp = oracle.run(kind, g, T)
    plan = Plan(Stencil(kind, shape), T)
    xs = [torch.from_numpy(g).cuda() for _ in range(2)]
    outs = [torch.empty_like(xs[0]) for _ in range(2)]
    for it in range(4):
        for k in range(2):
            outs[k].fill_(-7)
            plan.run(xs[k], outs[k])
            torch.cuda.synchronize()
            assert_bitexact(outs[k].cpu().numpy(), exp, f"{kind} run {it} set {k}")
            assert_bitexact(xs[k].cpu().numpy(), g, f"{kind} input untouched run {it}")
    for it in range(3):  # in place: the input is reset before each run
        y = torch.from_numpy(g).cuda() if it == 0 else y.copy_(torch.from_numpy(g))
        plan.run(y, out=y)
        torch.cuda.synchronize()
        assert_bitexact(y.cpu().numpy(), exp, f"{kind} in place run {it}")


def test_graph_replay_fdtd():
    f = stencil_inputs.fields((130, 260), seed=23, n=3)
    exp = oracle.fdtd(*f, 14)
    plan = Plan(Stencil("fdtd2d", f[0].shape), 14)
    for it in range(4):
        xs = [torch.from_numpy(a).cuda() for a in f]
        outs = [torch.empty_like(x) for x in xs]
        plan.run(xs, outs)
        torch.cuda.synchronize()
        for a, b in zip(outs, exp):
            assert_bitexact(a.cpu().numpy(), b, f"fdtd run {it}")


def test_output_tensors_validated():
    """Plan.run rejects output tensors that stencil_run would write out of bounds through."""
    from paper_conf_cgo_grosserchsv14_b200 import StencilError

    g = torch.from_numpy(stencil_inputs.uniform((64, 96), seed=1)).cuda()
    plan = Plan(Stencil("star2d5", (64, 96)), 4)
    bad = [torch.empty((64, 95), device="cuda"), torch.empty((64, 96), dtype=torch.float64, device="cuda"),
           torch.empty((96, 64), device="cuda").t(), torch.empty((64, 96))]
    for o in bad:
        with pytest.raises(StencilError):
            plan.run(g, o)


LIN_CASES = [
    # 13-point star of radius 2, upwind (one-sided) of radius 2, a 3D radius-2 access set, and
    # the 19-point 3D star-plus-edges of radius 1
    ([(0, 0), (-1, 0), (1, 0), (0, -1), (0, 1), (-2, 0), (2, 0), (0, -2), (0, 2)],
     [0.5, 0.1, 0.1, 0.1, 0.1, 0.025, 0.025, 0.025, 0.025], (67, 130), 13),
    ([(0, 0), (0, -1), (0, -2), (-1, 0)], [0.25, 0.5, 0.125, 0.125], (50, 75), 11),
    ([(0, 0, 0), (-2, 0, 0), (2, 0, 0), (0, -1, 0), (0, 1, 0), (0, 0, -2), (0, 0, 2), (1, 1, 1)],
     [0.3, 0.1, 0.1, 0.1, 0.1, 0.1, 0.1, 0.1], (19, 21, 26), 7),
    ([(0, 0, 0)] + [o for o in __import__("itertools").product((-1, 0, 1), repeat=3) if 0 < sum(map(abs, o)) <= 2],
     [0.25] + [0.75 / 18] * 18, (17, 20, 23), 6),
]


@pytest.mark.parametrize("dtype", [np.float32, np.float64])
@pytest.mark.parametrize("executor", ["auto", "naive"])
@pytest.mark.parametrize("case", range(len(LIN_CASES)))
def test_linear_stencils(case, executor, dtype):
    """General linear stencils (any access set and radius: general delta, the generic hybrid
    executor and the naive comparator) bit-exact against the oracle's plain loop."""
    offs, coefs, shape, T = LIN_CASES[case]
    g = stencil_inputs.uniform(shape, seed=40 + case, dtype=dtype)
    st = Stencil("linear", shape, dtype=dtype, offsets=offs, coefficients=coefs)
    plan = Plan(st, T, executor=executor)
    out = plan.run(torch.from_numpy(g).cuda())
    torch.cuda.synchronize()
    assert_bitexact(out.cpu().numpy(), oracle.linear(g, offs, coefs, T), f"linear case {case} {executor}")


@pytest.mark.parametrize("kind,ext,T,P,pd,fused,mode", [
    ("star3d7", (40, 64, 72), 23, 2, 1, "1", "fused"), ("star3d7", (33, 70, 132), 17, 3, 1, "1", "fused"),
    ("star3d7", (33, 70, 132), 17, 3, 1, "0", "p2p"), ("star3d7", (60, 40, 64), 19, 2, 0, "1", "p2p"),
    ("star2d5", (300, 512), 29, 3, -1, "1", "p2p"), ("box3d27", (30, 52, 64), 13, 2, 1, "1", "fused"),
    ("gradient3d", (21, 80, 68), 9, 4, 1, "1", "fused")])
def test_dist_loopback_device_initiated_halo(kind, ext, T, P, pd, fused, mode):
    """The device-initiated halo exchange (csrc/dist.cpp exchange_p2p, kernels/halo.cu) between P
    ranks that are plans of one process on this GPU (HEXS_DIST_LOOPBACK=1; tools/loop_check.py,
    in a subprocess with eager module loading): every rank's send kernel stores its halo lines
    into its neighbours' receive areas and publishes a sequence number, their wait kernels
    acquire it -- each rank on its own stream, all enqueued before any completes.  The gathered
    owned slabs must be bit-identical to the single-domain oracle, twice (the sequence numbers
    continue across runs)."""
    import os
    import subprocess
    import sys

    root = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
    env = dict(os.environ, CUDA_MODULE_LOADING="EAGER", HEXS_DIST_FUSED=fused)
    r = subprocess.run([sys.executable, os.path.join(root, "tools", "loop_check.py"), kind, ",".join(map(str, ext)),
                        str(T), str(P), str(pd)], env=env, capture_output=True, text=True, timeout=180)
    assert r.returncode == 0 and r.stdout.startswith("OK"), r.stdout + r.stderr[-2000:]
    assert f"exchange={mode}" in r.stdout, r.stdout
