"""One search on all SMs (the latency view): device us per iteration for C1..C4 (developer probe)."""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_ipps_luongmt10_b200 as L
import ppp_inputs as pi

for cfg, iters in (("C1", 2000), ("C2", 2000), ("C3", 2000), ("C4", 2000)):
    c = pi.CONFIGS[cfg]
    inst = pi.config_instance(cfg)
    with L.Instance(inst.A, inst.S) as I:
        best = 1e30
        for rep in range(3):
            L.lns_tabu_run(I.ctx, c["k"], iters, -1, pi.config_seed(cfg), None, 0)
            best = min(best, L.lns_last_kernel_ms(I.ctx))
    print(f"{cfg} single search: {1e3 * best / iters:.2f} us/iteration")
