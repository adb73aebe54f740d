import sys, os, numpy as np, torch
sys.path.insert(0, os.getcwd())
import oracle, stencil_inputs
from paper_conf_cgo_grosserchsv14_b200 import Plan, Stencil
for shape, T in (((70, 150, 140), 13), ((130, 90, 200), 17)):
    g = stencil_inputs.uniform(shape, seed=2)
    p = Plan(Stencil("star3d7", shape), T, h=3, w0=7, w=[16])
    out = p.run(torch.from_numpy(g).cuda()); torch.cuda.synchronize()
    exp = oracle.run("star3d7", g, T)
    print(shape, T, p.info.get("executor"), p.info.get("variant"), "bit-exact" if np.array_equal(out.cpu().numpy(), exp) else "MISMATCH")
