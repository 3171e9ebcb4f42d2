cp tools/variants/lib_trace.so paper_conf_asplos_ginsbachrsbdo18_b200/libspmv_b200.so
SPMV_GRAPH=0 python - <<'PY' 2>&1 | grep -v "^NCCL" | head -40
import os, sys, socket
sys.path.insert(0, ".")
import torch, torch.distributed as dist
import gen, paper_conf_asplos_ginsbachrsbdo18_b200 as sp
s = socket.socket(); s.bind(("127.0.0.1", 0)); port = s.getsockname()[1]; s.close()
dist.init_process_group("gloo", init_method=f"tcp://127.0.0.1:{port}", rank=0, world_size=1)
dev = torch.device("cuda:0")
A = gen.makea("S")
rp, ci, va = (torch.from_numpy(a).to(dev) for a in (A.rowptr, A.colidx, A.vals))
b = torch.from_numpy(gen.uniform(A.n, seed=3)).to(dev)
d = sp.Dist(0, 1, 0, transport="p2p")
M = sp.CSRMatrix(rp, ci, va, A.n, dist=d, kernel="xplan")
print(M.info())
x = torch.empty_like(b)
try:
    print(M.cg_solve(b, x, 1))
except Exception as e:
    print("ERR", e)
torch.cuda.synchronize()
PY
