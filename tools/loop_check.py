"""The device-initiated halo exchange between P ranks that are plans of this one process on this
one GPU (HEXS_DIST_LOOPBACK=1), checked bit for bit against the oracle:

    CUDA_MODULE_LOADING=EAGER python tools/loop_check.py KIND N0,N1[,N2] T P PART_DIM

Every rank runs on its own stream and all are enqueued before any completes: the wait kernels of
one rank spin until its neighbours' send kernels have published.  Eager module loading is needed
here (and only here): with lazy loading, the first launch of a kernel while another stream's
kernel spins on this process's device waits for the device to drain -- a deadlock that cannot
happen across processes (one rank per GPU).  Exit 0 = bit-identical for two consecutive runs."""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
os.environ["HEXS_DIST_LOOPBACK"] = "1"
import numpy as np  # noqa: E402
import torch  # noqa: E402

import oracle  # noqa: E402  (test infrastructure: the checker)
import stencil_inputs  # noqa: E402
from paper_conf_cgo_grosserchsv14_b200 import dist as hdist  # noqa: E402


def main(kind, ext, T, P, pd):
    uid = os.urandom(128)
    plans = [hdist.DistPlan(kind, ext, T, part_dim=pd, rank=r, nranks=P, unique_id=uid) for r in range(P)]
    g = stencil_inputs.uniform(ext, seed=11)
    exp = oracle.run(kind, g, T)
    locs = [p.scatter(g) for p in plans]
    outs = [torch.empty_like(x) for x in locs]
    streams = [torch.cuda.Stream() for _ in range(P)]
    torch.cuda.synchronize()
    for it in range(2):
        for p, x, o, s in zip(plans, locs, outs, streams):
            p.run(x, o, stream=s)
        torch.cuda.synchronize()
        got = np.concatenate([p.owned(o).cpu().numpy() for p, o in zip(plans, outs)], axis=plans[0].layout.part_dim)
        if not np.array_equal(got, exp):
            bad = np.argwhere(got != exp)
            print(f"MISMATCH run {it}: {len(bad)} values, first {tuple(bad[0])}", flush=True)
            return 1
    print(f"OK {kind} {ext} T={T} P={P} part_dim={plans[0].layout.part_dim} "
          f"launches={plans[0].launches_per_run} exchange={plans[0].exchange}", flush=True)
    return 0


if __name__ == "__main__":
    a = sys.argv[1:]
    sys.exit(main(a[0], tuple(int(v) for v in a[1].split(",")), int(a[2]), int(a[3]), int(a[4])))
