"""Timing experiment for the fast 3D kernel: python tools/mode3d.py [config [h w0]].
Mode 1 skips the progress counters (results are WRONG) to measure the synchronisation cost."""
import ctypes
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import bench  # noqa: E402
from paper_conf_cgo_grosserchsv14_b200 import Plan, Stencil, lib  # noqa: E402

cfg = sys.argv[1] if len(sys.argv) > 1 else "heat3d"
tile = {"h": int(sys.argv[2]), "w0": int(sys.argv[3])} if len(sys.argv) > 3 else {}
kind, ext, T, _ = bench.CONFIGS[cfg]
g = bench.make_inputs(kind, ext)[0]
plan = Plan(Stencil(kind, ext), T, **tile)
x = torch.from_numpy(g).cuda()
o = torch.empty_like(x)
L = lib()
L.hexs_debug_fast3d_mode.argtypes = [ctypes.c_int]
ups = plan.info["updates"]
for mode in [int(m) for m in os.environ.get("MODES", "0 1 0").split()]:
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
    print("%s h,w0=%s mode %d: %.2f ms/run  %.0f GUp/s" % (cfg, tile, mode, ms, ups / ms / 1e6), flush=True)
L.hexs_debug_fast3d_mode(0)
