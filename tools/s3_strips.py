"""Streaming 3D kernel: GUp/s vs the number of x strips per hexagon (carry pipeline depth)."""
import json, os, sys
import torch
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import stencil_inputs  # noqa: E402
from paper_conf_cgo_grosserchsv14_b200 import Plan, Stencil  # noqa: E402
T = 24
for N0, N1, N2 in [(512, 512, 36), (512, 512, 100), (512, 512, 164), (512, 512, 292), (512, 512, 512),
                   (512, 2048, 36), (512, 1024, 100)]:
    g = torch.from_numpy(stencil_inputs.uniform((N0, N1, N2), seed=0)).cuda()
    out = torch.empty_like(g)
    plan = Plan(Stencil("star3d7", (N0, N1, N2)), T, hex_dim=1)
    for _ in range(2):
        plan.run(g, out)
    torch.cuda.synchronize()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    e0.record()
    for _ in range(3):
        plan.run(g, out)
    e1.record()
    torch.cuda.synchronize()
    ms = e0.elapsed_time(e1) / 3
    info = plan.info
    print(json.dumps({"ext": [N0, N1, N2], "kernel": plan.executor_name, "ms": ms,
                      "gups": info["updates"] / ms / 1e6, "launches": info["n_launches"]}), flush=True)
