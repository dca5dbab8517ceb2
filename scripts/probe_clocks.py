"""The bench job repeated for ~3 s with nvidia-smi sampling clocks, power and throttle reasons
(developer probe: is a kernel variant power- or clock-limited?)."""
import os
import sys
import time

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np

import paper_conf_ipps_luongmt10_b200 as L
import ppp_inputs as pi
from bench import ClockSampler

inst = pi.config_instance("C4")
V0 = np.stack([pi.start_vector(117, pi.restart_seed(5, r)) for r in range(50)])
with L.Instance(inst.A, inst.S) as I:
    L.lns_tabu_run_batch(I.ctx, 3, 50, 400, -1, 0, V0, 0)
    with ClockSampler(0) as clk:
        ms = []
        t = time.time()
        while time.time() - t < 3.0:
            L.lns_tabu_run_batch(I.ctx, 3, 50, 400, -1, 0, V0, 0)
            ms.append(L.lns_last_kernel_ms(I.ctx))
    print(f"kernel ms min {min(ms):.2f} median {sorted(ms)[len(ms) // 2]:.2f} runs {len(ms)}", clk.summary())
