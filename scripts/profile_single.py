"""One C4 search of 1,000 iterations on all SMs (the latency view) for ncu: a warm-up launch,
then the profiled one."""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_ipps_luongmt10_b200 as L
import ppp_inputs as pi

inst = pi.config_instance("C4")
with L.Instance(inst.A, inst.S) as I:
    for rep in range(2):
        L.lns_tabu_run(I.ctx, 3, 1000, -1, 5, None, 0)
        print(rep, L.lns_last_kernel_ms(I.ctx))
