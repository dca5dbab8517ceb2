import sys, os
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np, torch
import paper_conf_ipps_luongmt10_b200 as L, ppp_inputs as pi
from math import comb
inst = pi.config_instance("C5"); n = 1024; k = int(sys.argv[1])
V = pi.start_vector(n, pi.config_seed("C5"))
M = comb(n, k)
ctx = L.lns_create(inst.A, inst.S)
Y = (inst.A.astype(np.int32) @ V.astype(np.int32)).astype(np.int32)
print("eval_neighborhood with true Y:", L.lns_eval_neighborhood(ctx, k, V, Y))
out = torch.empty(M, dtype=torch.int32, device="cuda")
L.lns_eval_all(ctx, k, V, out)
rng = np.random.default_rng(0)
ranks = np.unique(rng.integers(0, M, 2000))
got = out[torch.from_numpy(ranks).cuda()].cpu().numpy().astype(np.int64)
os.makedirs("gpurun_out", exist_ok=True)
np.savez(f"gpurun_out/c5diff_k{k}.npz", ranks=ranks, got=got)
print("saved")
