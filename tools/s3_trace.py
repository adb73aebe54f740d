"""Event trace of the streaming 3D kernel (debug build lib/libhexstencil_s3t.so):
HEXS_LIB=paper_conf_cgo_grosserchsv14_b200/lib/libhexstencil_s3t.so python tools/s3_trace.py
Runs one stencil_run of a 512^3 heat-3D problem (T = 6: the launches are full hexagons), then
prints per-strip step times and handoff latencies of the last launch."""
import ctypes, os, sys
import numpy as np
import torch
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import stencil_inputs  # noqa: E402
from paper_conf_cgo_grosserchsv14_b200 import Plan, Stencil, _lib  # noqa: E402

N2 = int(sys.argv[1]) if len(sys.argv) > 1 else 512
T = int(sys.argv[2]) if len(sys.argv) > 2 else 6
g = torch.from_numpy(stencil_inputs.uniform((512, 512, N2), seed=0)).cuda()
plan = Plan(Stencil("star3d7", g.shape), T, hex_dim=1)
os.environ["HEXS_NO_GRAPH"] = "1"
out = plan.run(g)
torch.cuda.synchronize()
L = _lib.lib()
fn = getattr(L, "hexs_s3_trace_v0")
buf = np.zeros((512, 16, 1200), dtype=np.uint64)
assert fn(buf.ctypes.data_as(ctypes.c_void_p)) == 0
info = plan.info
nstr = (N2 - 1 + 4 * (info["H"] - 1)) // 64 + 1
last = plan.launches()[-1]
nitems = (last["S0_hi"] - last["S0_lo"] + 1) * nstr
print("strips", nstr, "items", nitems)
t = buf[:nitems].astype(np.int64)
n = 512 - 2 + last["a_hi"] - last["a_lo"] + 2
t0 = t[:, 0, 0].min()
print("launch", last, "n_steps", n, "span us", (t[:, 0, n - 1].max() - t0) / 1e3)
for it in list(range(min(nitems, 2 * nstr))):
    done = t[it, 0, :n]
    d = np.diff(done)
    pub_lag = t[it, 1, :n] - t[it, 0, :n]
    pred = t[it, 2, :n] - t[max(it - 1, 0), 1, :n] if it % nstr else np.zeros(n)
    issued = t[it, 3, :n] - t[it, 2, :n] if it % nstr else np.zeros(n)
    wait = t[it, 0, 1:n] - t[it, 3, 1:n] if it % nstr else np.zeros(1)
    big = np.argsort(d)[-3:]
    print(f"item {it:3d} strip {it % nstr}: start {(done[0]-t0)/1e3:7.1f}us end {(done[-1]-t0)/1e3:8.1f}us "
          f"step med {np.median(d):5.0f} mean {np.mean(d):6.0f} max {d.max():7.0f} at {list(big)} | pub lag {np.median(pub_lag):5.0f} "
          f"| pred seen after pub {np.median(pred):6.0f} | issue {np.median(issued):4.0f} | done-after-issue {np.median(wait):6.0f}")
st = (t[:, 0, 0] - t0) / 1e3
en = (t[:, 0, n - 1] - t0) / 1e3
order = np.argsort(st)
print("start/end per item (us), by start:")
for k in range(0, nitems, 9):
    print(" ".join(f"{int(i)}:{st[i]:.0f}-{en[i]:.0f}" for i in order[k:k + 9]))

print("phase means per item (ns): start->full_x, full_x->full_c, compute, barrier+tail")
for it in range(nitems):
    a = t[it]
    ph = [np.mean(a[5, 2:n-2] - a[4, 2:n-2]), np.mean(a[6, 2:n-2] - a[5, 2:n-2]), np.mean(a[7, 2:n-2] - a[6, 2:n-2]),
          np.mean(a[0, 2:n-2] - a[7, 2:n-2]), np.mean(a[4, 3:n-1] - a[0, 2:n-2])]
    if it % 3 == 0:
        print(f"item {it:3d} strip {it % nstr} end {en[it]:6.0f}: " + " ".join(f"{x:7.0f}" for x in ph))

print("per-warp 'ready for barrier' time relative to step start (tid 0 stamp 4), mean ns, warps 0..5")
for it in range(0, nitems, 3):
    a = t[it]
    w = [np.mean(a[8 + k, 2:n-2] - a[4, 2:n-2]) for k in range(6)]
    print(f"item {it:3d} strip {it % nstr} end {en[it]:6.0f}: " + " ".join(f"{x:7.0f}" for x in w))
