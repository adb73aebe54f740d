"""Timing experiment for the fast 3D kernel: python tools/mode3d.py [h w0].

Runs the heat3d config with the kernel's debug modes (0 = normal, 1 = no carries,
2 = no In planes, 3 = neither; results are WRONG in modes 1-3) to split the step time
into compute-bound and load/handoff-bound parts."""
import ctypes
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import bench  # noqa: E402
from paper_conf_cgo_grosserchsv14_b200 import Plan, Stencil, lib  # noqa: E402

tile = {}
if len(sys.argv) > 2:
    tile = {"h": int(sys.argv[1]), "w0": int(sys.argv[2])}
kind, ext, T, _ = bench.CONFIGS["heat3d"]
g = bench.make_inputs(kind, ext)[0]
plan = Plan(Stencil(kind, ext), T, **tile)
x = torch.from_numpy(g).cuda()
o = torch.empty_like(x)
L = lib()
L.hexs_debug_fast3d_mode.argtypes = [ctypes.c_int]
ups = float(g.size) * T
for mode in [int(m) for m in os.environ.get('MODES', '0 1 2 3 0').split()]:
    L.hexs_debug_fast3d_mode(mode)
    plan.run(x, o)
    torch.cuda.synchronize()
    s, e = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    s.record()
    for _ in range(3):
        plan.run(x, o)
    e.record()
    torch.cuda.synchronize()
    ms = s.elapsed_time(e) / 3
    print("mode %d: %.2f ms/run  %.0f GUp/s" % (mode, ms, ups / ms / 1e6))
L.hexs_debug_fast3d_mode(0)
