"""Small runs of every kernel family for compute-sanitizer (memcheck / racecheck / synccheck):
persistent search (one and several CTAs), batched restarts, stepped search, eval_all, unranking."""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np

import paper_conf_ipps_luongmt10_b200 as L
import ppp_inputs as pi

c1 = pi.config_instance("C1")
with L.Instance(c1.A, c1.S) as I:
    I.tabu_run(1, 40, -1, seed=3, stop_on_zero=False)
    L.lns_tabu_run_batch(I.ctx, 1, 4, 30, -1, 5, None, 0)
small = pi.planted_instance(40, 45, 123)
V = pi.start_vector(45, 9)
ctx = L.lns_create(small.A, small.S, 0)
try:
    for k in (2, 3):
        L.lns_eval_all(ctx, k, V)
    L.lns_config(ctx, 2)
    L.lns_tabu_run(ctx, 3, 6, -1, 1, None, 0)
    L.lns_tabu_run(ctx, 2, 6, -1, 1, None, L.LNS_FORCE_STEPPED)
    L.lns_tabu_run_batch(ctx, 3, 3, 4, -1, 7, None, 0)
    L.lns_tabu_run(ctx, 2, 8, 3, 1, None, L.LNS_TABU_SOLUTIONS)  # solution list: scan + group barrier
    L.lns_tabu_run_batch(ctx, 1, 2, 8, 2, 7, None, L.LNS_TABU_SOLUTIONS)
    L.lns_tabu_run(ctx, 4, 4, -1, 1, None, 0)  # k > 3: k_gen, several CTAs
    L.lns_eval_all(ctx, 5, V)
    L.lns_tabu_run_batch(ctx, 4, 3, 3, -1, 2, None, 0)  # k > 3 batched restarts
finally:
    L.lns_destroy(ctx)
big = pi.planted_instance(260, 40, 5)  # m > 255: segment-loop path, padded placement
with L.Instance(big.A, big.S) as I:
    L.lns_config(I.ctx, 1)
    I.tabu_run(3, 4, -1, seed=2, stop_on_zero=False)
from ppp_inputs import bqp as bi  # the UBQP kernels: eval, apply, init, graph replay

bq = L.lns_bqp_create(bi.random_q(70, 0.3, 1), 0)
try:
    xq = bi.start_x(70, 2)
    for k in (1, 2, 3):
        L.lns_bqp_eval_all(bq, k, xq)
    L.lns_bqp_tabu_run(bq, 3, 130, -1, xq)  # two graph blocks of 64 + 2 direct iterations
    L.lns_bqp_tabu_run(bq, 2, 10, 3, xq)
finally:
    L.lns_bqp_destroy(bq)
print("sanitize probe done")
