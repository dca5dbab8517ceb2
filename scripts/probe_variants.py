"""Developer probe: cost of the tabu-list variants on C4, one search on all SMs
and the bench's batched job (50 searches x 400 iterations). Not the bench (no L2 flush, no clocks)."""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np

import paper_conf_ipps_luongmt10_b200 as L
import ppp_inputs as pi

inst = pi.config_instance("C4")
M = L.lns_neighborhood_size(117, 3)
V0s = np.stack([pi.start_vector(117, pi.restart_seed(5, r)) for r in range(50)])
with L.Instance(inst.A, inst.S) as I:
    for name, fl in (("rank list (default)", 0), ("aspiration", L.LNS_ASPIRATION),
                     ("solution list", L.LNS_TABU_SOLUTIONS)):
        for rep in range(2):
            L.lns_tabu_run(I.ctx, 3, 2000, -1, 6, None, fl)
            ms1 = L.lns_last_kernel_ms(I.ctx)
            L.lns_tabu_run_batch(I.ctx, 3, 50, 400, -1, 0, V0s, fl)
            msb = L.lns_last_kernel_ms(I.ctx)
        print(f"{name:22s} single: {1000 * ms1 / 2000:7.2f} us/iteration ({2000 * M / ms1 * 1e3:.3e} nbr/s)"
              f"   batch 50x400: {msb:7.2f} ms ({50 * 400 * M / msb * 1e3:.3e} nbr/s)")
