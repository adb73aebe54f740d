"""Cycle accounting of the 3D phase kernel (debug build): where do the CTAs spend time?

  python native_build.py --timing        # builds lib/libhexstencil_tm.so (-DHEXS_F3_TIMING)
  HEXS_LIB=.../libhexstencil_tm.so python tools/f3_timing.py CONFIG [h w0 [wy]]

Prints, for thread 0 (TMA issuer) and thread 64 (compute-only warp), the share of cycles
per category summed over all CTAs of one stencil_run: mbarrier (TMA) wait, CTA barrier,
predecessor-flag spin, compute, TMA issue."""
import ctypes
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import numpy as np  # noqa: E402
import torch  # noqa: E402

import bench  # noqa: E402
from paper_conf_cgo_grosserchsv14_b200 import Plan, Stencil, _lib  # noqa: E402

cfg = sys.argv[1] if len(sys.argv) > 1 else "heat3d"
tile = {}
if len(sys.argv) > 3:
    tile = {"h": int(sys.argv[2]), "w0": int(sys.argv[3])}
if len(sys.argv) > 4:
    tile["w"] = (int(sys.argv[4]), 0, 0)
kind, ext, T, _ = bench.CONFIGS[cfg]
plan = Plan(Stencil(kind, ext), T, **tile)
x = torch.from_numpy(bench.make_inputs(kind, ext)[0]).cuda()
y = torch.empty_like(x)
lib = _lib.lib()
fns = [getattr(lib, f"hexs_f3_timing_v{i}") for i in range(64) if hasattr(lib, f"hexs_f3_timing_v{i}")]
buf = (ctypes.c_ulonglong * (1024 * 2 * 8))()


def collect(reset_only=False):
    tot = np.zeros((1024, 2, 8))
    for fn in fns:  # only the variant the plan runs has non-zero counters
        fn(buf, 1)
        tot += np.frombuffer(buf, dtype=np.uint64).reshape(1024, 2, 8).astype(np.float64)
    return tot


plan.run(x, y)
torch.cuda.synchronize()
collect()
plan.run(x, y)
torch.cuda.synchronize()
a = collect()
names = ["mbar_wait", "cta_barrier", "flag_spin", "compute", "tma_issue"]
for t, who in enumerate(["thread0 (issuer)", "thread64 (compute)"]):
    s = a[:, t, :5].sum(axis=0)
    tot = s.sum()
    print(who, " ".join(f"{n}={100 * v / tot:.1f}%" for n, v in zip(names, s)), f"total={tot:.3e} cycles")
