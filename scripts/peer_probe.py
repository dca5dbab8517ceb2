"""Per-iteration cost of the device-initiated exchange (f3) on one GPU: P partitions x nb CTAs
exchanging through each other's buffers (plain launches, concurrent streams) vs one context with
P*nb CTAs, and vs the host-stepped path (eval launch + apply launch per iteration, no collective)."""
import os, sys, threading, time
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np, torch
import paper_conf_ipps_luongmt10_b200 as L, ppp_inputs as pi

cfg = sys.argv[1] if len(sys.argv) > 1 else "C4"
iters = int(sys.argv[2]) if len(sys.argv) > 2 else 500
c = pi.CONFIGS[cfg]; inst = pi.config_instance(cfg); k = c["k"]
V0 = torch.from_numpy(pi.start_vector(inst.n, pi.config_seed(cfg))).cuda()


def single(nb, flags=0):
    ctx = L.lns_create(inst.A, inst.S); L.lns_config(ctx, nb)
    L.lns_tabu_run(ctx, k, iters, -1, 0, V0, flags)
    t = time.perf_counter(); L.lns_tabu_run(ctx, k, iters, -1, 0, V0, flags); w = time.perf_counter() - t
    ms = L.lns_last_kernel_ms(ctx); L.lns_destroy(ctx)
    return 1e3 * ms / iters, 1e6 * w / iters


def peers(P, nb):
    ctxs = [L.lns_create(inst.A, inst.S) for _ in range(P)]
    for cx in ctxs:
        L.lns_config(cx, nb); L.lns_tabu_run(cx, k, iters, -1, 0, V0, 0)
    bufs = [L.lns_exchange_buffer(cx) for cx in ctxs]
    for p, cx in enumerate(ctxs):
        L.lns_attach_peers(cx, p, P, bufs, 20000)
    streams = [torch.cuda.Stream() for _ in ctxs]
    walls = []
    for rep in range(2):
        for cx in ctxs:
            L.lns_exchange_reset(cx)
        def run(p):
            L.lns_tabu_run(ctxs[p], k, iters, -1, 0, V0, L.LNS_PLAIN_LAUNCH, stream=streams[p])
        t = time.perf_counter()
        th = [threading.Thread(target=run, args=(p,)) for p in range(P)]
        [x.start() for x in th]; [x.join() for x in th]
        walls.append(time.perf_counter() - t)
    ms = max(L.lns_last_kernel_ms(cx) for cx in ctxs)
    for cx in ctxs:
        L.lns_destroy(cx)
    return 1e3 * ms / iters, 1e6 * walls[-1] / iters


for nb_total in (32, 64, 128):
    s_k, s_w = single(nb_total)
    line = f"{cfg} {nb_total:3d} CTAs: one context {s_k:6.2f} us/iter"
    for P in (2, 4):
        p_k, p_w = peers(P, nb_total // P)
        line += f" | {P} partitions x {nb_total // P}: {p_k:6.2f} us/iter (wall {p_w:6.2f})"
    st_k, st_w = single(nb_total, L.LNS_FORCE_STEPPED)
    line += f" | host-stepped: {st_w:6.2f} us/iter (wall)"
    print(line, flush=True)
