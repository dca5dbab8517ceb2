"""One bench step (C4, 50 runs x 400 iterations, batched) for ncu: warm-up step, then the profiled one."""
import os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import paper_conf_ipps_luongmt10_b200 as L, ppp_inputs as pi
inst = pi.config_instance("C4")
ctx = L.lns_create(inst.A, inst.S)
for s in range(2):
    V0 = np.stack([pi.start_vector(117, pi.restart_seed(5 + s, r)) for r in range(50)])
    res = L.lns_tabu_run_batch(ctx, 3, 50, 400, -1, 0, V0, 0)
    print(s, L.lns_last_kernel_ms(ctx), sum(r["iters_done"] for r in res))
