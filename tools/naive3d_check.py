"""Naive 3D comparator: parity on small grids and its GUp/s / HBM bandwidth at 512^3 and 1024^3."""
import json, os, sys
import numpy as np
import torch
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import oracle  # noqa: E402
import stencil_inputs  # noqa: E402
from paper_conf_cgo_grosserchsv14_b200 import Plan, Stencil  # noqa: E402
for kind in ("star3d7", "gradient3d"):
    for shape, T in [((20, 37, 68), 5), ((70, 9, 132), 3)]:
        g = stencil_inputs.uniform(shape, seed=3)
        out = Plan(Stencil(kind, shape), T, executor="naive").run(torch.from_numpy(g).cuda()).cpu().numpy()
        assert np.array_equal(out, oracle.run(kind, g, T)), (kind, shape)
print("naive parity ok")
for N, T in [(512, 128), (1024, 16)]:
    g = torch.from_numpy(stencil_inputs.uniform((N, N, N), seed=0)).cuda()
    o = torch.empty_like(g)
    plan = Plan(Stencil("star3d7", (N, N, N)), T, executor="naive")
    for _ in range(2):
        plan.run(g, o)
    torch.cuda.synchronize()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    e0.record(); plan.run(g, o); e1.record(); torch.cuda.synchronize()
    ms = e0.elapsed_time(e1)
    up = (N - 2) ** 3 * T
    print(json.dumps({"N": N, "T": T, "naive_gups": up / ms / 1e6, "gbs_at_8B": up * 8 / ms / 1e6}))
