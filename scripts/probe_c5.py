"""C5 (1024 x 1024, 3-Hamming): one search of 5 iterations and 8 batched restarts x 3 iterations;
device time and device memory the library holds (developer probe)."""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_ipps_luongmt10_b200 as L
import ppp_inputs as pi

inst = pi.config_instance("C5")
M = L.lns_neighborhood_size(1024, 3)
with L.Instance(inst.A, inst.S) as I:
    for rep in range(2):
        L.lns_tabu_run(I.ctx, 3, 5, -1, 6, None, 0)
    ms = L.lns_last_kernel_ms(I.ctx)
    print(f"C5 single: {ms / 5:.2f} ms/iteration, {5 * M / ms * 1e3:.3e} nbr/s, pool live {L.lns_pool_stats()[1] / 1e6:.0f} MB")
    for rep in range(2):
        L.lns_tabu_run_batch(I.ctx, 3, 8, 3, -1, 1005, None, 0)
    ms = L.lns_last_kernel_ms(I.ctx)
    print(f"C5 8 restarts x 3: {ms:.1f} ms, {24 * M / ms * 1e3:.3e} nbr/s, pool live {L.lns_pool_stats()[1] / 1e6:.0f} MB")
