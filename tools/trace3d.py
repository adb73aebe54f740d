"""Timeline of one fast3d launch (debug): python tools/trace3d.py [launch_index]."""
import ctypes, os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np, torch
import bench
from paper_conf_cgo_grosserchsv14_b200 import Plan, Stencil, lib
li = int(sys.argv[1]) if len(sys.argv) > 1 else 10
kind, ext, T, _ = bench.CONFIGS["heat3d"]
g = bench.make_inputs(kind, ext)[0]
plan = Plan(Stencil(kind, ext), T)
x = torch.from_numpy(g).cuda(); o = torch.empty_like(x)
tr = torch.zeros(200000 * 32, dtype=torch.int64, device="cuda")
L = lib(); L.hexs_debug_fast3d_trace.argtypes = [ctypes.c_void_p, ctypes.c_int64]
L.hexs_debug_fast3d_trace(ctypes.c_void_p(tr.data_ptr()), li)
plan.run(x, o); torch.cuda.synchronize()
L.hexs_debug_fast3d_trace(None, -1)
t = tr.view(-1, 32).cpu().numpy()
n = int((t[:, 1] > 0).sum()); t = t[:n]
t0 = t[:, 1].min()
rel = (t[:, 1:] - t0) / 1e3
print("items", n, "launch span us", (t[:, 2:].max() - t0) / 1e3)
L_ = plan.info["H"]
pro = rel[:, 1] - rel[:, 0]
print("prologue wait us: mean %.2f p90 %.2f" % (pro.mean(), np.percentile(pro, 90)))
for k in range(L_):
    f, d, c = rel[:, 2 + 3 * k], rel[:, 3 + 3 * k], rel[:, 4 + 3 * k]
    prev = rel[:, 1] if k == 0 else rel[:, 4 + 3 * (k - 1)]
    if k == 0:
        print("level 0 compute us: mean %.2f" % (c - prev).mean())
        continue
    ok = f > 0
    print("level %d: flag wait %.2f  data wait %.2f  compute %.2f (us, mean)" % (
        k, (f - prev)[ok].mean(), (d - f)[ok].mean(), (c - d)[ok].mean()))
tot = rel[:, 4 + 3 * (L_ - 1)] - rel[:, 0]
print("per item total us: mean %.2f; items per CTA-slot %.1f" % (tot.mean(), n / 296))
np.save(os.path.join(os.path.dirname(os.path.dirname(os.path.abspath(__file__))), "gpurun_out", "trace3d.npy"), t)
