"""One C4 (or given cfg) tabu search for ncu: a warm-up launch then the profiled launch."""
import os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_ipps_luongmt10_b200 as L, ppp_inputs as pi
cfg = sys.argv[1] if len(sys.argv) > 1 else "C4"
iters = int(sys.argv[2]) if len(sys.argv) > 2 else 100
c = pi.CONFIGS[cfg]; inst = pi.config_instance(cfg)
ctx = L.lns_create(inst.A, inst.S)
for s in range(2):
    print(L.lns_tabu_run(ctx, c["k"], iters, -1, 5 + s, None, 0), L.lns_last_kernel_ms(ctx))
