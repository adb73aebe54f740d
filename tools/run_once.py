"""Run one config's hot path a few times (for ncu captures): python tools/run_once.py CONFIG [RUNS] [h w0]."""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import bench  # noqa: E402
from paper_conf_cgo_grosserchsv14_b200 import Plan, Stencil  # noqa: E402

cfg = sys.argv[1] if len(sys.argv) > 1 else "heat2d5"
runs = int(sys.argv[2]) if len(sys.argv) > 2 else 2
tile = {}
if len(sys.argv) > 4:
    tile = {"h": int(sys.argv[3]), "w0": int(sys.argv[4])}
execu = os.environ.get("HEXS_EXEC", "auto")
kind, ext, T, _ = bench.CONFIGS[cfg][:4]
fields = bench.make_inputs(kind, ext)
plan = Plan(Stencil(kind, ext), T, executor=execu, **tile)
xs = [torch.from_numpy(f).cuda() for f in fields]
outs = [torch.empty_like(x) for x in xs]
for _ in range(runs):
    plan.run(xs[0] if len(xs) == 1 else xs, outs[0] if len(xs) == 1 else outs)
torch.cuda.synchronize()
print(cfg, plan.info["n_launches"], "launches per run")
