"""Fig. 8 ladder: 1-Hamming tabu search on instances
m x n = (100t+1) x (100t+17), t = 1..15, 10,000 iterations each; GPU time vs the CPU oracle
(timed on a bounded number of iterations and scaled, as the paper scaled its 3-Hamming CPU times).
The paper reports the GPU acceleration factor growing from x1.1 at 201x217 to x10.8 at 1501x1517."""
import argparse, json, os, sys, time
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_ipps_luongmt10_b200 as L
import ppp_inputs as pi


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--iters", type=int, default=10000)
    ap.add_argument("--cpu-iters", type=int, default=200)
    ap.add_argument("--tmax", type=int, default=15)
    ap.add_argument("--out", default="results/fig8_r01.json")
    a = ap.parse_args()
    import oracle
    rows = []
    for t in range(1, a.tmax + 1):
        m, n = 100 * t + 1, 100 * t + 17
        inst = pi.planted_instance(m, n, 3000 + t)
        with L.Instance(inst.A, inst.S) as I:
            L.lns_tabu_run(I.ctx, 1, 50, -1, 1, None, 0)
            res = L.lns_tabu_run(I.ctx, 1, a.iters, -1, 2, None, 0)
            gms = L.lns_last_kernel_ms(I.ctx)
        V0 = pi.start_vector(n, 2)
        c0 = time.perf_counter()
        oracle.tabu_run(inst.A, inst.S, 1, V0, a.cpu_iters, n // 6, stop_on_zero=False)
        cpu_s = (time.perf_counter() - c0) * a.iters / a.cpu_iters
        row = {"t": t, "m": m, "n": n, "iters": a.iters, "gpu_s": gms / 1e3, "gpu_us_per_iter": gms * 1e3 / a.iters,
               "cpu_oracle_s_scaled": cpu_s, "cpu_threads": oracle.max_threads(), "speedup_vs_oracle": cpu_s / (gms / 1e3),
               "row_evals_per_s": a.iters * n * m / (gms / 1e3), "final_f": res["final_f"]}
        rows.append(row)
        print(f"{m}x{n}: GPU {gms/1e3:7.3f} s ({row['gpu_us_per_iter']:6.1f} us/iter)  oracle {cpu_s:8.2f} s "
              f"({row['cpu_threads']} thr, scaled from {a.cpu_iters})  x{row['speedup_vs_oracle']:6.1f}  "
              f"{row['row_evals_per_s']:.2e} row-evals/s", flush=True)
    os.makedirs(os.path.dirname(a.out) or ".", exist_ok=True)
    json.dump({"protocol": "Fig. 8 (PAPER.md:270-364): 1-Hamming TS, 10,000 iterations", "rows": rows}, open(a.out, "w"), indent=1)


if __name__ == "__main__":
    main()
