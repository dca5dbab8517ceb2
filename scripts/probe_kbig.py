"""Developer probe: k = 4, 5 (the generic-k kernel) on the paper's shapes, one
search on the GPU vs the CPU oracle (a few iterations)."""
import os
import sys
import time

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import oracle
import paper_conf_ipps_luongmt10_b200 as L
import ppp_inputs as pi

for (m, n, k, iters, cpu_iters) in ((73, 73, 4, 50, 2), (101, 117, 4, 20, 1), (73, 73, 5, 10, 1), (81, 81, 5, 5, 1)):
    inst = pi.planted_instance(m, n, 6000 + m + k)
    M = L.lns_neighborhood_size(n, k)
    with L.Instance(inst.A, inst.S) as I:
        I.tabu_run(k, 3, -1, seed=1, stop_on_zero=False)
        res = I.tabu_run(k, iters, -1, seed=2, stop_on_zero=False)[3]
        ms = L.lns_last_kernel_ms(I.ctx)
    V0 = pi.start_vector(n, 2)
    c0 = time.perf_counter()
    oracle.tabu_run(inst.A, inst.S, k, V0, cpu_iters, M // 6, stop_on_zero=False)
    cpu = (time.perf_counter() - c0) / cpu_iters
    print(f"{m}x{n} k={k}: M={M} GPU {1000 * ms / iters:9.1f} us/iteration = {iters * M / ms * 1e3:.3e} nbr/s"
          f" (row-evals {iters * M * m / ms * 1e3:.3e}/s); oracle {cpu * 1e3:8.1f} ms/iteration"
          f" ({oracle.max_threads() if hasattr(oracle, 'max_threads') else '?'} threads) x{cpu / (ms / iters / 1000):.0f}")
