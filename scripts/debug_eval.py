"""Debug helper: eval_all of one shape vs the oracle, per state; prints the first mismatches."""
import os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
sys.path.insert(0, os.path.join(os.path.dirname(os.path.dirname(os.path.abspath(__file__))), "tests"))
import numpy as np
import paper_conf_ipps_luongmt10_b200 as L, ppp_inputs as pi, oracle as orc
from test_gpu_parity import _states
m, n, k = (int(x) for x in sys.argv[1:4])
inst = pi.planted_instance(m, n, 7000 + m * 31 + n)
rng = np.random.default_rng(m * n + k)
ctx = L.lns_create(inst.A, inst.S)
for si, V in enumerate(_states(inst, rng, count=2)):
    got = L.lns_eval_all(ctx, k, V).astype(np.int64)
    want = orc.eval_all(inst.A, inst.S, V, k)
    bad = np.nonzero(got != want)[0]
    Y = inst.A.astype(np.int64) @ V.astype(np.int64)
    vals, cnts = np.unique(Y, return_counts=True)
    print(f"state {si}: {len(bad)} / {len(want)} wrong; Y range [{Y.min()},{Y.max()}], max segment {cnts.max()}")
    for r in bad[:5]:
        print("   rank", r, "got", got[r], "want", want[r], "diff", got[r] - want[r])
L.lns_destroy(ctx)
