import sys, os
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np, torch
import paper_conf_ipps_luongmt10_b200 as L, ppp_inputs as pi, oracle
from math import comb
shapes = [(int(a), int(b), int(k)) for a, b, k in (s.split("x") for s in sys.argv[1].split(","))]
for m, n, k in shapes:
    if os.environ.get("C5"):
        inst = pi.config_instance("C5"); V = pi.start_vector(n, pi.config_seed("C5"))
    else:
        inst = pi.planted_instance(m, n, 77); V = pi.start_vector(n, 3)
    M = comb(n, k)
    ctx = L.lns_create(inst.A, inst.S)
    out = torch.empty(M, dtype=torch.int32, device="cuda")
    L.lns_eval_all(ctx, k, V, out)
    rng = np.random.default_rng(0)
    ranks = np.unique(rng.integers(0, M, 300))
    got = out[torch.from_numpy(ranks).cuda()].cpu().numpy().astype(np.int64)
    want = oracle.eval_ranks(inst.A, inst.S, V, k, ranks)
    Y = inst.A.astype(int) @ V
    print(f"{m}x{n} k={k}: mismatches {int((got != want).sum())}/{len(ranks)} diff sample {(got - want)[:6]} vmin {Y.min()} vmax {Y.max()}", flush=True)
    L.lns_destroy(ctx)
