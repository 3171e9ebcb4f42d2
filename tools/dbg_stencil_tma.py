"""One stencil27_apply call on an nx x ny x nz grid (fp64, default path), compared to the oracle."""
import os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
sys.path.insert(0, os.path.join(os.path.dirname(os.path.dirname(os.path.abspath(__file__))), "tests"))
import numpy as np, torch
import gen, oracle
import paper_conf_asplos_ginsbachrsbdo18_b200 as sp
nx, ny, nz = map(int, sys.argv[1:4])
n = nx * ny * nz
xh = gen.uniform(n, seed=1)
x = torch.from_numpy(xh).cuda(); y = torch.zeros_like(x)
sp.stencil27_apply(nx, ny, nz, x, y)
torch.cuda.synchronize()
yr, b = oracle.stencil27(nx, ny, nz, xh)
print(nx, ny, nz, "maxerr", float(np.max(np.abs(y.cpu().numpy() - yr))), flush=True)
