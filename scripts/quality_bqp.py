"""UBQP analogue of the paper's quality protocol (Tabs. I-III: larger k
gives better solutions at a fixed iteration budget): OR-Library-style instances (n = 200, density
0.1, entries in [-100, 100]), 5 starts each, k = 1, 2, 3, the same number of iterations for every k,
default tenure floor(C(n,k)/6). Writes results/quality_bqp_r01.md. DESIGN.md §5.13."""
import os
import sys
import time

import numpy as np

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_ipps_luongmt10_b200 as L  # noqa: E402
from ppp_inputs import bqp as bi  # noqa: E402

N, DENS, INST, STARTS, ITERS = 200, 0.1, 10, 5, 2000
rows = []
best_of = {}
for s in range(INST):
    Q = bi.random_q(N, DENS, 1000 + s)
    ctx = L.lns_bqp_create(Q, 0)
    for k in (1, 2, 3):
        bests, ms = [], 0.0
        for q in range(STARTS):
            _, _, _, res = L.lns_bqp_tabu_run(ctx, k, ITERS, -1, bi.start_x(N, 50 * s + q), trace=False)
            bests.append(res["best_f"])
            ms += L.lns_bqp_last_kernel_ms(ctx)
        best_of[(s, k)] = bests
        rows.append((s, k, float(np.mean(bests)), int(min(bests)), ms / STARTS))
    L.lns_bqp_destroy(ctx)
    print(s, [r[2] for r in rows[-3:]], flush=True)

lines = ["# UBQP quality vs k (round 1)", "",
         f"`scripts/quality_bqp.py`: {INST} instances `random_q({N}, {DENS}, 1000 + s)`, {STARTS} starts each "
         f"(`start_x(n, 50 s + q)`), {ITERS} iterations for every k, tenure floor(C(n,k)/6). One B200; device "
         "time per run. Best fitness per run (lower is better); `best found in this experiment` = the least over all 15 runs "
         "of the instance.", "",
         "| instance | best found in this experiment | k=1 mean / min | k=2 mean / min | k=3 mean / min | ms per run k=1 / 2 / 3 |",
         "|---|---|---|---|---|---|"]
hits = {1: 0, 2: 0, 3: 0}
for s in range(INST):
    bk = min(min(best_of[(s, k)]) for k in (1, 2, 3))
    r = {k: next(x for x in rows if x[0] == s and x[1] == k) for k in (1, 2, 3)}
    for k in (1, 2, 3):
        hits[k] += sum(b == bk for b in best_of[(s, k)])
    lines.append(f"| {s} | {bk} | " + " | ".join(f"{r[k][2]:.1f} / {r[k][3]}" for k in (1, 2, 3)) +
                 " | " + " / ".join(f"{r[k][4]:.1f}" for k in (1, 2, 3)) + " |")
lines += ["", "Runs reaching the best value found in this experiment (of " + str(INST * STARTS) + "): " +
          ", ".join(f"k={k}: {hits[k]}" for k in (1, 2, 3)), ""]
os.makedirs("results", exist_ok=True)
open("results/quality_bqp_r01.md", "w").write("\n".join(lines))
print("\n".join(lines))
