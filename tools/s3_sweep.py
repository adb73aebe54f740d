"""Time the streaming 3D kernel (and the tile-wavefront one) over tiles on the bench grids.
python tools/s3_sweep.py [kind] [N] [T]  -> one JSON line per (kernel, h, w0)."""
import json
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import stencil_inputs  # noqa: E402
from paper_conf_cgo_grosserchsv14_b200 import Plan, Stencil  # noqa: E402

kind = sys.argv[1] if len(sys.argv) > 1 else "star3d7"
N = int(sys.argv[2]) if len(sys.argv) > 2 else 512
T = int(sys.argv[3]) if len(sys.argv) > 3 else 128
tiles = [(2, 7, 1), (1, 7, 1), (2, 5, 1), (3, 5, 1), (3, 7, 1), (1, 3, 1), (3, 7, 0), (0, 0, 1)]
if kind == "gradient3d":
    tiles = [(2, 7, 1), (1, 7, 1), (2, 7, 0)]
g = torch.from_numpy(stencil_inputs.uniform((N, N, N), seed=0)).cuda()
out = torch.empty_like(g)
st = Stencil(kind, (N, N, N))
for h, w0, hd in tiles:
    try:
        plan = Plan(st, T, h=h, w0=w0, hex_dim=hd)
    except Exception as e:  # noqa: BLE001
        print(json.dumps({"h": h, "w0": w0, "hex_dim": hd, "error": str(e)}), flush=True)
        continue
    for _ in range(3):
        plan.run(g, out)
    torch.cuda.synchronize()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    e0.record()
    for _ in range(5):
        plan.run(g, out)
    e1.record()
    torch.cuda.synchronize()
    ms = e0.elapsed_time(e1) / 5
    info = plan.info
    print(json.dumps({"kind": kind, "N": N, "T": T, "h": info["h"], "w0": info["w0"], "hex_dim": info["hex_dim"],
                      "kernel": plan.executor_name, "ms": ms, "gups": info["updates"] / ms / 1e6,
                      "launches": info["n_launches"]}), flush=True)
