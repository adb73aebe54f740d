"""Event timeline of the 3D phase kernel (debug build with -DHEXS_F3_TRACE).

  python -c "import native_build as n, os; n.EXTRA3D[:] = ['-DHEXS_F3_TRACE']; \
             n.build_library(lib=os.path.join(n.PKG, 'lib', 'libhexstencil_tr.so'))"
  HEXS_LIB=.../libhexstencil_tr.so python tools/f3_trace.py [CONFIG]

For CTAs 0..7 of the first launches of one stencil_run: per level, the compute threads' wait
(full-barrier wait + level barrier) and compute time, and the producer's empty-wait, flag-wait
and fill issue points, in SM cycles."""
import ctypes
import os
import sys
from collections import defaultdict

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import numpy as np  # noqa: E402
import torch  # noqa: E402

import bench  # noqa: E402
from paper_conf_cgo_grosserchsv14_b200 import Plan, Stencil, _lib  # noqa: E402

cfg = sys.argv[1] if len(sys.argv) > 1 else "heat3d"
kind, ext, T, _ = bench.CONFIGS[cfg]
plan = Plan(Stencil(kind, ext), T)
x = torch.from_numpy(bench.make_inputs(kind, ext)[0]).cuda()
y = torch.empty_like(x)
lib = _lib.lib()
fns = [getattr(lib, f"hexs_f3_trace_v{i}") for i in range(64) if hasattr(lib, f"hexs_f3_trace_v{i}")]
buf = (ctypes.c_ulonglong * (8 * 8192))()
cnt = (ctypes.c_int * 8)()
plan.run(x, y)
torch.cuda.synchronize()
for fn in fns:
    fn(buf, cnt, 1)
plan.run(x, y)
torch.cuda.synchronize()
ev = None
for fn in fns:
    fn(buf, cnt, 1)
    if max(cnt) > 0:
        ev = np.frombuffer(buf, dtype=np.uint64).reshape(8, 8192).copy()
        counts = list(cnt)
        break
names = {1: "p_empty_wait", 2: "p_fill", 3: "p_flag0", 4: "p_flag1", 5: "c_wait", 6: "c_start", 7: "c_end", 8: "c_tile_end"}
agg = defaultdict(list)
for c in range(8):
    n = min(counts[c], 8192)
    e = ev[c, :n]
    typ = (e >> 60).astype(int)
    tile = ((e >> 44) & 0xFFFF).astype(int)
    lev = ((e >> 36) & 0xFF).astype(int)
    clk = (e & 0xFFFFFFFFF).astype(np.int64)
    # one launch (tile counter restarts at every launch): LAUNCH = 1 is the first full-time
    # launch (launch 0 is cut by t = 0); segments end at the tile-0 ends of consecutive launches
    seen0 = list(np.where((typ == 8) & (tile == 0))[0])
    cuts = [0] + [j + 1 for j in seen0]
    L0 = int(os.environ.get("LAUNCH", "1"))
    start = cuts[L0] if L0 < len(cuts) else 0
    stop = cuts[L0 + 1] if L0 + 1 < len(cuts) else n
    last = {}
    for i in range(start, stop):
        t, k, a, ck = typ[i], tile[i], lev[i], clk[i]
        last[(t, k, a)] = ck
        if t == 6 and (5, k, a) in last:
            agg[("wait", a)].append(ck - last[(5, k, a)])
        if t == 7 and (6, k, a) in last:
            agg[("compute", a)].append(ck - last[(6, k, a)])
        if t == 4 and (3, k, a) in last:
            agg[("flag", a)].append(ck - last[(3, k, a)])
        if t == 2 and (1, k, a) in last:
            agg[("p_emptywait+issue", a)].append(ck - last[(1, k, a)])
        if t == 6 and (2, k, a) in last:
            agg[("fill_to_start", a)].append(ck - last[(2, k, a)])
    if c == 0:
        print("CTA 0, first 2 tiles:")
        for i in range(start, min(stop, start + 60)):
            print(f"  {names[typ[i]]:18s} tile {tile[i]:3d} level {lev[i]} t={clk[i] - clk[start]:9d}")
print("per level, cycles (mean over CTAs 0-7, launch", os.environ.get("LAUNCH", "1"), "):")
for key in sorted(agg):
    v = np.array(agg[key])
    print(f"  {key[0]:20s} level {key[1]}: mean {v.mean():8.0f}  median {np.median(v):8.0f}  n={len(v)}")
