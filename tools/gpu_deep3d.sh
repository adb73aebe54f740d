#!/bin/bash
# deeper / wider hexagons with 16 x 64 tiles: (4,7), (3,9) against (3,7)
tag=${1:-dp}
mkdir -p gpurun_out
cat > /tmp/deep_check.py <<'PY'
import os, sys, numpy as np, torch
sys.path.insert(0, os.getcwd())
import oracle, stencil_inputs
from paper_conf_cgo_grosserchsv14_b200 import Plan, Stencil
for h, w0 in ((4, 7), (3, 9)):
    for shape, T in (((70, 150, 140), 23), ((40, 90, 300), 9)):
        g = stencil_inputs.uniform(shape, seed=5)
        p = Plan(Stencil("star3d7", shape), T, h=h, w0=w0, w=[16])
        out = p.run(torch.from_numpy(g).cuda()); torch.cuda.synchronize()
        print((h, w0), shape, T, p.info.get("w"), "bit-exact" if np.array_equal(out.cpu().numpy(), oracle.run("star3d7", g, T)) else "MISMATCH", flush=True)
PY
timeout 300 python /tmp/deep_check.py > gpurun_out/${tag}_check.log 2>&1
for t in 4,7,16 3,9,16 3,7,16; do
  timeout 300 python bench.py --config heat3d --no-cpu --tile $t >> gpurun_out/${tag}_heat3d.json 2>> gpurun_out/${tag}.err
done
