"""Debug aid: the loopback device-initiated exchange, with host-side progress prints."""
import os
import sys
import time

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
os.environ["HEXS_DIST_LOOPBACK"] = "1"
import torch  # noqa: E402

import stencil_inputs  # noqa: E402
from paper_conf_cgo_grosserchsv14_b200 import dist as hdist  # noqa: E402

kind, ext, T, P, pd = sys.argv[1], tuple(int(v) for v in sys.argv[2].split(",")), int(sys.argv[3]), int(sys.argv[4]), int(sys.argv[5])
uid = os.urandom(128)
plans = [hdist.DistPlan(kind, ext, T, part_dim=pd, rank=r, nranks=P, unique_id=uid) for r in range(P)]
print("created", [p.layout for p in plans], flush=True)
g = stencil_inputs.uniform(ext, seed=11)
locs = [p.scatter(g) for p in plans]
outs = [torch.empty_like(x) for x in locs]
streams = [torch.cuda.Stream() for _ in range(P)]
torch.cuda.synchronize()
print("launches per run", plans[0].launches_per_run, flush=True)
for r in range(P):
    print("enqueue", r, flush=True)
    plans[r].run(locs[r], outs[r], stream=streams[r])
    print("enqueued", r, flush=True)
for i in range(20):
    q = [s.query() for s in streams]
    print(i, q, flush=True)
    if all(q):
        break
    time.sleep(1)
os._exit(0)
