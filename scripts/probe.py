"""Developer probe: time lns_tabu_run per configuration (not the bench; no L2 flush, no clocks)."""
import argparse
import os
import sys
import time

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))

import numpy as np
import torch

import paper_conf_ipps_luongmt10_b200 as L
import ppp_inputs as pi


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--cfg", default="C1,C2,C3,C4,C5")
    ap.add_argument("--blocks", default="0")
    ap.add_argument("--iters", type=int, default=0)
    ap.add_argument("--stepped", action="store_true")
    a = ap.parse_args()
    for cfg in a.cfg.split(","):
        c = pi.CONFIGS[cfg]
        inst = pi.config_instance(cfg)
        iters = a.iters or c["iters"]
        if cfg == "C5":
            iters = min(iters, 3)
        M = L.lns_neighborhood_size(inst.n, c["k"])
        with L.Instance(inst.A, inst.S) as I:
            for nb in [int(x) for x in a.blocks.split(",")]:
                L.lns_config(I.ctx, nb)
                flags = L.LNS_FORCE_STEPPED if a.stepped else 0
                L.lns_tabu_run(I.ctx, c["k"], min(iters, 50), -1, 1, None, flags)
                torch.cuda.synchronize()
                t = time.perf_counter()
                res = L.lns_tabu_run(I.ctx, c["k"], iters, -1, pi.config_seed(cfg), None, flags)
                wall = time.perf_counter() - t
                ms = L.lns_last_kernel_ms(I.ctx)
                it = res["iters_done"]
                print(f"{cfg} blocks={nb} iters={it} kernel_ms={ms:.3f} wall_ms={wall*1e3:.2f} "
                      f"us/iter={ms*1e3/max(it,1):.2f} iters/s={it/(ms/1e3):.0f} "
                      f"nbr/s={it*M/(ms/1e3):.3e} final_f={res['final_f']} best_f={res['best_f']}", flush=True)


if __name__ == "__main__":
    main()
