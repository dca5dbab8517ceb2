"""Time the UBQP tabu search on a few shapes: device time of lns_bqp_tabu_run."""
import os
import sys
from math import comb

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_ipps_luongmt10_b200 as L  # noqa: E402
from ppp_inputs import bqp as bi  # noqa: E402

for k, n, dens, iters in [(1, 2500, 0.1, 2000), (2, 500, 0.1, 1000), (2, 2500, 0.1, 100), (3, 117, 0.1, 1000),
                          (3, 250, 0.1, 200), (3, 500, 0.1, 50)]:
    Q = bi.random_q(n, dens, 1)
    ctx = L.lns_bqp_create(Q, 0)
    x0 = bi.start_x(n, 2)
    L.lns_bqp_tabu_run(ctx, k, min(iters, 64), -1, x0, trace=False)
    _, _, _, res = L.lns_bqp_tabu_run(ctx, k, iters, -1, x0, trace=False)
    ms = L.lns_bqp_last_kernel_ms(ctx)
    M = comb(n, k)
    print(f"k={k} n={n} M={M} iters={iters}: {ms / iters * 1e3:.2f} us/iteration, "
          f"{M * iters / ms * 1e3:.3e} neighbours/s, best_f {res['best_f']}", flush=True)
    L.lns_bqp_destroy(ctx)
