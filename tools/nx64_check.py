"""Bit-exact check of the wide 3D tile variants (NX = 64 / 128) against the oracle on ragged grids:
python tools/nx64_check.py (GPU)."""
import os
import sys

import numpy as np
import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import oracle  # noqa: E402
import stencil_inputs  # noqa: E402
from paper_conf_cgo_grosserchsv14_b200 import Plan, Stencil  # noqa: E402

ok = True
for kind, h, w0, wy in (("star3d7", 3, 7, 16), ("star3d7", 3, 7, 8), ("star3d7", 2, 7, 16), ("box3d27", 2, 7, 16),
                        ("gradient3d", 2, 7, 16)):
    for shape, T in (((70, 150, 140), 13), ((40, 90, 300), 9)):
        g = stencil_inputs.uniform(shape, seed=2)
        p = Plan(Stencil(kind, shape), T, h=h, w0=w0, w=[wy])
        out = p.run(torch.from_numpy(g).cuda())
        torch.cuda.synchronize()
        exp = oracle.run(kind, g, T)
        same = np.array_equal(out.cpu().numpy(), exp)
        ok &= same
        print(kind, (h, w0, wy), shape, T, p.info.get("w"), "bit-exact" if same else "MISMATCH", flush=True)
print("ALL OK" if ok else "FAILURES")
