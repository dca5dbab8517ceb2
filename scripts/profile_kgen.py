"""One k = 4 search (73 x 73, the generic-k kernel k_gen) for ncu: a warm-up launch, then the profiled one."""
import os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_ipps_luongmt10_b200 as L, ppp_inputs as pi
inst = pi.planted_instance(73, 73, 6077)
with L.Instance(inst.A, inst.S) as I:
    for s in range(2):
        print(I.tabu_run(4, 20, -1, seed=2 + s, stop_on_zero=False)[3], L.lns_last_kernel_ms(I.ctx))
