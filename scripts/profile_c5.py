"""C5 under ncu: one search of 3 iterations (one k_search launch), then 8 batched restarts x 3
iterations (one launch). Used with --metrics dram__bytes_read.sum,dram__bytes_write.sum."""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_ipps_luongmt10_b200 as L
import ppp_inputs as pi

inst = pi.config_instance("C5")
with L.Instance(inst.A, inst.S) as I:
    L.lns_tabu_run(I.ctx, 3, 3, -1, 6, None, 0)
    L.lns_tabu_run_batch(I.ctx, 3, 8, 3, -1, 1005, None, 0)
    print("ok", L.lns_last_kernel_ms(I.ctx))
