"""Time fast-2D variants that differ in warps per CTA (chunk width w1 = NW*128 fp32 columns):
python tools/nw_sweep.py kind h w0 w1 [w1 ...]   (8192^2, T=512, kernel-region CUDA events)"""
import json
import sys

import torch

sys.path.insert(0, __import__("os").path.dirname(__import__("os").path.dirname(__import__("os").path.abspath(__file__))))
from paper_conf_cgo_grosserchsv14_b200 import Plan, Stencil  # noqa: E402

kind, h, w0 = sys.argv[1], int(sys.argv[2]), int(sys.argv[3])
N, T = 8192, 512
x = torch.rand((N, N), device="cuda")
out = torch.empty_like(x)
for w1 in [int(v) for v in sys.argv[4:]]:
    p = Plan(Stencil(kind, (N, N)), T, h=h, w0=w0, w=(w1, 0, 0))
    p.run(x, out=out)
    p.run(x, out=out)
    torch.cuda.synchronize()
    p.profile(3)
    for _ in range(3):
        p.run(x, out=out)
    torch.cuda.synchronize()
    ms = p.profile_read()["kernel_ms"] / 3
    print(json.dumps({"kind": kind, "h": h, "w0": w0, "w1": p.info["w"][0], "ms": ms,
                      "gups": (N - 2) ** 2 * T / ms / 1e6}), flush=True)
