import os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np, torch
import stencil_inputs
from paper_conf_cgo_grosserchsv14_b200 import Plan, Stencil
shape = (30, 37, 68); T = int(sys.argv[1]) if len(sys.argv) > 1 else 2
g = stencil_inputs.uniform(shape, seed=30)
p = Plan(Stencil("star3d7", shape), T)
print(p.info["fast_kernel"], p.info["n_launches"], p.launches()[:3])
x = torch.from_numpy(g).cuda()
o = p.run(x)
torch.cuda.synchronize()
import oracle
print("ok", np.array_equal(o.cpu().numpy(), oracle.run("star3d7", g, T)))
