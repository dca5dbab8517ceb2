#!/usr/bin/env python
"""Benchmark of the B200 k-Hamming tabu search.

Contract: ``python bench.py --gpus N --steps K --warmup W [--impl reference]`` prints ONE JSON
line on rank 0. Workload (BASELINE.json ``metric``: "PPP 3-Hamming neighbors evaluated/sec and
tabu iters/sec at 1/2/4/8 B200", quoted at 1/2/4/8 GPUs on configs[3]): the planted PPP instance
m = 101, n = 117 (seed 1004), 3-Hamming neighbourhood (C(117,3) = 260,130 neighbours), tabu
tenure floor(M/6) = 43,355, no early stop. One STEP = one tabu search of 2,000 iterations
(every iteration evaluates all 260,130 neighbours, selects, moves) from the start vector of seed
5 + step. With N > 1 the rank space is partitioned across the GPUs and one NCCL u64-MIN
all-reduce per iteration picks the global move (strong scaling: the total work is fixed).

``value`` = neighbours evaluated per second over the whole job (device time, CUDA events, max
over ranks), inputs already resident in HBM. ``e2e`` = the same metric through the C ABI with
HOST buffers (instance upload, start vector, trace and final vector copies inside the timed
region). ``roofline`` = the persistent search kernel's integer throughput against the issue-rate
peak derived in DESIGN.md §6. ``cpu_baseline`` = the CPU oracle timed on this host on a bounded
sample. ``--impl reference`` times that oracle alone as the reference arm.
"""
from __future__ import annotations

import argparse
import json
import os
import statistics
import subprocess
import sys
import tempfile
import time
from math import comb

ROOT = os.path.dirname(os.path.abspath(__file__))
sys.path.insert(0, ROOT)

import numpy as np  # noqa: E402

import ppp_inputs as pi  # noqa: E402

METRIC = "PPP 3-Hamming neighbors evaluated/sec and tabu iters/sec at 1/2/4/8 B200"
UNIT = "neighbors/s"
CFG = "C4"
ITERS = 2000
L2_FLUSH_BYTES = 512 << 20  # > 126 MB L2


def env_int(name, default):
    try:
        return int(os.environ.get(name, default))
    except ValueError:
        return default


def peaks():
    try:
        with open(os.path.join(ROOT, "MEASURED_PEAKS.json")) as fh:
            return json.load(fh), "measured"
    except OSError:
        return {"sm_max_mhz": 1965.0, "hbm_gbs": 6650.0}, "fallback"


class ClockSampler:
    """nvidia-smi clocks and throttle reasons sampled every 50 ms during the timed region."""

    FIELDS = ["clocks.sm", "clocks.max.sm", "power.draw", "clocks_event_reasons.hw_slowdown",
              "clocks_event_reasons.hw_thermal_slowdown", "clocks_event_reasons.sw_thermal_slowdown",
              "clocks_event_reasons.sw_power_cap"]

    def __init__(self, gpu_index: int):
        self.gpu = gpu_index
        self.proc = None
        self.path = None

    def __enter__(self):
        fd, self.path = tempfile.mkstemp(suffix=".csv")
        os.close(fd)
        try:
            self.proc = subprocess.Popen(
                ["nvidia-smi", f"--query-gpu={','.join(self.FIELDS)}", "--format=csv,noheader,nounits",
                 "-lms", "50", "-i", str(self.gpu)], stdout=open(self.path, "w"), stderr=subprocess.DEVNULL)
        except OSError:
            self.proc = None
        time.sleep(0.3)
        return self

    def __exit__(self, *exc):
        if self.proc is not None:
            self.proc.terminate()
            try:
                self.proc.wait(timeout=5)
            except subprocess.TimeoutExpired:
                self.proc.kill()

    def summary(self):
        rows = []
        try:
            with open(self.path) as fh:
                for line in fh:
                    p = [x.strip() for x in line.split(",")]
                    if len(p) == len(self.FIELDS):
                        rows.append(p)
        except OSError:
            pass
        finally:
            try:
                os.unlink(self.path)
            except OSError:
                pass
        if not rows:
            return {"sm_mhz": None, "sm_max_mhz": None, "reasons": ["unavailable"], "samples": 0}
        sm = [float(r[0]) for r in rows if r[0].replace(".", "").isdigit()]
        loaded = [x for x in sm if x > 600] or sm
        names = ["hw_slowdown", "hw_thermal_slowdown", "sw_thermal_slowdown", "sw_power_cap"]
        reasons = sorted({names[i] for r in rows for i in range(4) if r[3 + i].lower().startswith("active")})
        return {"sm_mhz": statistics.median(loaded) if loaded else None,
                "sm_max_mhz": float(rows[0][1]) if rows[0][1].replace(".", "").isdigit() else None,
                "reasons": reasons, "samples": len(rows)}


# --------------------------------------------------------------------------------- oracle arm
def oracle_sample(budget_s: float, nthreads: int = 0):
    """Time the CPU oracle (as it stands) on the same instance / tenure, a bounded number of
    iterations sized to ~budget_s. Returns (neighbors/s, iters/s, iterations, cores, seconds)."""
    import oracle

    c = pi.CONFIGS[CFG]
    inst = pi.config_instance(CFG)
    M = comb(inst.n, c["k"])
    V0 = pi.start_vector(inst.n, pi.config_seed(CFG))
    ten = pi.default_tenure(inst.n, c["k"])
    t = time.perf_counter()
    oracle.tabu_run(inst.A, inst.S, c["k"], V0, 3, ten, stop_on_zero=False, nthreads=nthreads)
    per_iter = (time.perf_counter() - t) / 3
    iters = int(max(3, min(ITERS, budget_s / max(per_iter, 1e-6))))
    t = time.perf_counter()
    oracle.tabu_run(inst.A, inst.S, c["k"], V0, iters, ten, stop_on_zero=False, nthreads=nthreads)
    dt = time.perf_counter() - t
    cores = nthreads or oracle.max_threads()
    return iters * M / dt, iters / dt, iters, cores, dt


def run_reference(args, rank, world):
    """--impl reference: the CPU oracle (the only reference this paper has)."""
    if rank != 0:
        return
    import oracle

    oracle.build()
    c = pi.CONFIGS[CFG]
    inst = pi.config_instance(CFG)
    M = comb(inst.n, c["k"])
    ten = pi.default_tenure(inst.n, c["k"])
    per_step = 8  # iterations of the search per step (bounded sample of the 2,000-iteration step)
    times = []
    for s in range(args.warmup + args.steps):
        V0 = pi.start_vector(inst.n, 5 + s)
        t = time.perf_counter()
        oracle.tabu_run(inst.A, inst.S, c["k"], V0, per_step, ten, stop_on_zero=False)
        if s >= args.warmup:
            times.append(time.perf_counter() - t)
    total = sum(times)
    value = args.steps * per_step * M / total
    cores = oracle.max_threads()
    line = {
        "impl": "reference", "metric": METRIC, "value": value, "unit": UNIT, "n_gpus": args.gpus,
        "steps": args.steps, "warmup": args.warmup, "ms_per_step": 1e3 * total / args.steps,
        "higher_is_better": True, "scaling": "strong", "vs_baseline": None, "dtype": "int32",
        "data": "synthetic planted PPP instance (seeded splitmix64)",
        "config": {"workload": f"{CFG}: PPP m=101 n=117, 3-Hamming, tenure {ten}", "iters_per_step": per_step,
                   "parallelism": "cpu-openmp", "l2": "n/a (CPU)"},
        "tabu_iters_per_s": args.steps * per_step / total,
        "cpu_baseline": {"value": value, "unit": UNIT, "cores": cores, "kind": "oracle",
                         "sample": f"{per_step} tabu iterations of {CFG} per step from scratch (oracle, {cores} OpenMP threads)"},
        "e2e": {"value": value, "unit": UNIT, "h2d_bytes_per_step": 0, "d2h_bytes_per_step": 0},
    }
    print(json.dumps(line), flush=True)


# --------------------------------------------------------------------------------- GPU arm
def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--gpus", type=int, default=1)
    ap.add_argument("--steps", type=int, default=5)
    ap.add_argument("--warmup", type=int, default=3)
    ap.add_argument("--impl", default="lns", choices=["lns", "reference"])
    ap.add_argument("--iters", type=int, default=ITERS)
    ap.add_argument("--no-cpu-baseline", action="store_true")
    ap.add_argument("--cpu-budget", type=float, default=12.0)
    args = ap.parse_args()
    rank, world, local = env_int("RANK", 0), env_int("WORLD_SIZE", 1), env_int("LOCAL_RANK", 0)
    if args.impl == "reference":
        run_reference(args, rank, world)
        return
    args.warmup = max(args.warmup, 3)

    import torch
    import torch.distributed as dist

    import paper_conf_ipps_luongmt10_b200 as L

    torch.cuda.set_device(local)
    dev = torch.device("cuda", local)
    if world > 1:
        dist.init_process_group("nccl", device_id=dev)
    c = pi.CONFIGS[CFG]
    k = c["k"]
    inst = pi.config_instance(CFG)
    M = comb(inst.n, k)
    ten = pi.default_tenure(inst.n, k)
    iters = args.iters
    ctx = L.lns_create(inst.A, inst.S, local)
    if world > 1:
        pg = dist.distributed_c10d._get_default_group()
        comm = pg._get_backend(dev)._comm_ptr()
        L.lns_attach_comm(ctx, comm, rank, world)
    stream = torch.cuda.current_stream(dev)
    nsteps = args.warmup + args.steps
    V0s = torch.stack([torch.from_numpy(pi.start_vector(inst.n, 5 + s)) for s in range(nsteps)]).to(dev)
    tr = torch.empty(iters, dtype=torch.int64, device=dev)
    tf = torch.empty(iters, dtype=torch.int64, device=dev)
    Vo = torch.empty(inst.n, dtype=torch.int8, device=dev)
    flush = torch.empty(L2_FLUSH_BYTES // 4, dtype=torch.int32, device=dev)

    def step(s):
        return L.lns_tabu_run(ctx, k, iters, ten, 0, V0s[s], 0, Vo, tr, tf, stream)

    for s in range(args.warmup):
        step(s)
    torch.cuda.synchronize()
    ev0 = [torch.cuda.Event(enable_timing=True) for _ in range(args.steps)]
    ev1 = [torch.cuda.Event(enable_timing=True) for _ in range(args.steps)]
    kernel_ms, iters_done = [], 0
    with ClockSampler(local) as clk:
        for i in range(args.steps):
            flush.fill_(i)  # evict L2 between timed steps
            if world > 1:
                dist.barrier()
            torch.cuda.synchronize()
            ev0[i].record(stream)
            res = step(args.warmup + i)
            ev1[i].record(stream)
            torch.cuda.synchronize()
            kernel_ms.append(L.lns_last_kernel_ms(ctx))
            iters_done += res["iters_done"]
    clocks = clk.summary()
    step_ms = [a.elapsed_time(b) for a, b in zip(ev0, ev1)]
    total_ms = sum(step_ms)
    kern_ms = sum(kernel_ms)
    if world > 1:
        t = torch.tensor([total_ms, kern_ms], dtype=torch.float64, device=dev)
        dist.all_reduce(t, op=dist.ReduceOp.MAX)
        total_ms, kern_ms = float(t[0]), float(t[1])
    value = iters_done * M / (total_ms / 1e3)

    # ---- end to end through the C ABI with host buffers (pinned), same metric
    A_h = torch.from_numpy(inst.A).pin_memory()
    S_h = torch.from_numpy(inst.S).pin_memory()
    V0_h = torch.from_numpy(pi.start_vector(inst.n, 5)).pin_memory()
    tr_h = torch.empty(iters, dtype=torch.int64).pin_memory()
    tf_h = torch.empty(iters, dtype=torch.int64).pin_memory()
    Vo_h = torch.empty(inst.n, dtype=torch.int8).pin_memory()
    e2e_ms = 0.0
    e2e_iters = 0
    for i in range(args.steps):
        flush.fill_(i)
        if world > 1:
            dist.barrier()
        torch.cuda.synchronize()
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        e0.record(stream)
        c2 = L.lns_create(A_h, S_h, local)
        if world > 1:
            L.lns_attach_comm(c2, comm, rank, world)
        r2 = L.lns_tabu_run(c2, k, iters, ten, 0, V0_h, 0, Vo_h, tr_h, tf_h, stream)
        L.lns_destroy(c2)
        e1.record(stream)
        torch.cuda.synchronize()
        e2e_ms += e0.elapsed_time(e1)
        e2e_iters += r2["iters_done"]
    if world > 1:
        t = torch.tensor([e2e_ms], dtype=torch.float64, device=dev)
        dist.all_reduce(t, op=dist.ReduceOp.MAX)
        e2e_ms = float(t[0])
    e2e_value = e2e_iters * M / (e2e_ms / 1e3)
    h2d = A_h.numel() + 4 * S_h.numel() + V0_h.numel()
    d2h = 8 * tr_h.numel() + 8 * tf_h.numel() + Vo_h.numel()

    # ---- roofline: the persistent search kernel (one launch per step)
    pk, src = peaks()
    mhz = float(pk.get("sm_max_mhz", 1965.0))
    sms = torch.cuda.get_device_properties(dev).multi_processor_count
    ops_per_nbr = inst.m * (k + 4)  # SURVEY.md §8(d) model: k sign reads + Y' add + penalty + 2 histogram moves per row
    kern_avg_s = kern_ms / 1e3 / args.steps
    achieved = (iters * M / world) * ops_per_nbr / kern_avg_s / 1e12  # per-GPU share of the work
    peak = sms * 128 * mhz * 1e6 / 1e12  # 128 integer lanes issued per SM per clock (4 SMSP x 1 warp-instr)
    traffic = None
    prof = os.path.join(ROOT, "profiles", "r01_ncu_k_search_C4.json")  # ncu --set full of the bench step
    if os.path.exists(prof):
        try:
            with open(prof) as fh:
                traffic = json.load(fh).get("dram_bytes_per_launch")
        except (OSError, ValueError):
            traffic = None
    roofline = {"bound": "alu", "achieved": achieved, "peak": peak, "unit": "Tops/s", "frac": achieved / peak,
                "traffic": traffic, "kernel": "k_search<3> (persistent tabu search)",
                "peak_source": f"{sms} SMs x 128 int lanes/clk x {mhz:.0f} MHz ({src} sm_max_mhz)",
                "ops_per_neighbor": ops_per_nbr}

    cpu = None
    if rank == 0 and world == 1 and not args.no_cpu_baseline:
        v, ips, it, cores, dt = oracle_sample(args.cpu_budget)
        cpu = {"value": v, "unit": UNIT, "cores": cores, "kind": "oracle",
               "sample": f"{it} tabu iterations of {CFG} (same instance, tenure, start vector of seed 5), "
                         f"{dt:.1f} s, from-scratch fitness per neighbour", "tabu_iters_per_s": ips}
    if rank == 0:
        line = {
            "metric": METRIC, "value": value, "unit": UNIT, "n_gpus": world, "steps": args.steps,
            "warmup": args.warmup, "ms_per_step": total_ms / args.steps, "higher_is_better": True,
            "scaling": "strong", "vs_baseline": None, "dtype": "int32",
            "data": "synthetic planted PPP instance (seeded splitmix64, DESIGN.md §3)",
            "config": {"workload": f"{CFG}: PPP m=101 n=117, 3-Hamming (260,130 neighbours), tabu tenure {ten}, "
                                   f"{iters} iterations per step, no early stop",
                       "iters_per_step": iters, "parallelism": f"rank-space partition x{world}" if world > 1 else "1 GPU",
                       "l2": "flushed (512 MiB write) between timed steps"},
            "tabu_iters_per_s": iters_done / (total_ms / 1e3),
            "e2e": {"value": e2e_value, "unit": UNIT, "h2d_bytes_per_step": h2d, "d2h_bytes_per_step": d2h,
                    "tabu_iters_per_s": e2e_iters / (e2e_ms / 1e3)},
            # our kernels per timed step: 2 x k_fill_i64 + k_init + (1 persistent k_search | 2 per iteration stepped)
            "gpu_launches": args.steps * (4 if world == 1 else 2 + 2 * iters),
            "clocks": clocks,
            "roofline": roofline,
            "cpu_baseline": cpu,
        }
        print(json.dumps(line), flush=True)
    L.lns_destroy(ctx)
    if world > 1:
        dist.destroy_process_group()


if __name__ == "__main__":
    main()
