"""UBQP restarts: R searches one after another (lns_bqp_tabu_run) against one batched call
(lns_bqp_tabu_run_batch), device time (developer probe)."""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np

import paper_conf_ipps_luongmt10_b200 as L
from ppp_inputs import bqp as bi

for n, k, R, iters in [(200, 1, 50, 2000), (200, 2, 50, 2000), (200, 3, 50, 2000), (500, 3, 16, 256)]:
    Q = bi.random_q(n, 0.1, 1)
    X0 = np.stack([bi.start_x(n, 100 + r) for r in range(R)])
    ctx = L.lns_bqp_create(Q, 0)
    seq = 0.0
    L.lns_bqp_tabu_run(ctx, k, 128, -1, X0[0], trace=False)
    for r in range(R):
        L.lns_bqp_tabu_run(ctx, k, iters, -1, X0[r], trace=False)
        seq += L.lns_bqp_last_kernel_ms(ctx)
    L.lns_bqp_tabu_run_batch(ctx, k, X0, 128)
    L.lns_bqp_tabu_run_batch(ctx, k, X0, iters)
    bat = L.lns_bqp_last_kernel_ms(ctx)
    L.lns_bqp_destroy(ctx)
    M = L.lns_neighborhood_size(n, k)
    print(f"n={n} k={k} R={R} iters={iters}: one after another {seq:.1f} ms, batched {bat:.1f} ms "
          f"(x{seq / bat:.1f}), {R * iters * M / (bat / 1e3):.3e} neighbours/s batched", flush=True)
