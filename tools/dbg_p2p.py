import os, sys, socket
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np, torch, torch.distributed as dist
import gen, paper_conf_asplos_ginsbachrsbdo18_b200 as sp
s = socket.socket(); s.bind(("127.0.0.1", 0)); port = s.getsockname()[1]; s.close()
dist.init_process_group("gloo", init_method=f"tcp://127.0.0.1:{port}", rank=0, world_size=1)
dev = torch.device("cuda:0")
A = gen.makea("S")
rp, ci, va = (torch.from_numpy(a).to(dev) for a in (A.rowptr, A.colidx, A.vals))
b = torch.from_numpy(gen.uniform(A.n, seed=3)).to(dev)
for kernel in ("vector", "xplan", "merge"):
    res = {}
    for tr in ("single", "nccl", "p2p"):
        d = None if tr == "single" else sp.Dist(0, 1, 0, transport=tr)
        with sp.CSRMatrix(rp, ci, va, A.n, dist=d, kernel=kernel) as M:
            for k in (1, 2):
                x = torch.empty_like(b)
                try:
                    its, rn = M.cg_solve(b, x, k)
                except Exception as e:
                    its, rn = -1, str(e)[:80]
                res[(tr, k)] = (its, rn, float(x[:5].sum().item()))
        if d: d.close()
    for k, v in res.items(): print(kernel, k, v)
