"""One UBQP search (k = 3, n = 500) for ncu: 3 iterations, plain launches."""
import os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_ipps_luongmt10_b200 as L
from ppp_inputs import bqp as bi
Q = bi.random_q(500, 0.1, 1)
ctx = L.lns_bqp_create(Q, 0)
print(L.lns_bqp_tabu_run(ctx, 3, 3, -1, bi.start_x(500, 2), trace=False)[3], L.lns_bqp_last_kernel_ms(ctx))
L.lns_bqp_destroy(ctx)
