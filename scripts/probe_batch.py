"""Throughput of batched restarts (lns_tabu_run_batch) vs one search at a time."""
import os, sys, time
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_ipps_luongmt10_b200 as L, ppp_inputs as pi
for spec in sys.argv[1:]:
    parts = spec.split(":")
    cfg, R, iters = parts[0], int(parts[1]), int(parts[2])
    nbo = int(parts[3]) if len(parts) > 3 else 0  # CTAs per search override (0 = automatic)
    c = pi.CONFIGS[cfg]; inst = pi.config_instance(cfg)
    M = L.lns_neighborhood_size(inst.n, c["k"])
    with L.Instance(inst.A, inst.S) as I:
        L.lns_config(I.ctx, nbo)
        L.lns_tabu_run_batch(I.ctx, c["k"], min(R, 4), 5, -1, 1, None, 0)
        t = time.perf_counter()
        res = L.lns_tabu_run_batch(I.ctx, c["k"], R, iters, -1, 7, None, 0)
        wall = time.perf_counter() - t
        ms = L.lns_last_kernel_ms(I.ctx)
        it = sum(r["iters_done"] for r in res)
        solved = sum(r["solved"] for r in res)
        print(f"{cfg} R={R} nb={nbo} iters={iters} kernel_ms={ms:.1f} wall_ms={wall*1e3:.1f} agg_iters/s={it/(ms/1e3):.0f} "
              f"agg_nbr/s={it*M/(ms/1e3):.3e} solved={solved}/{R}", flush=True)
