"""Per-phase cycle breakdown of the persistent kernel (profiling build, LNS_LIB=liblns_prof.so)."""
import os, sys, ctypes
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
from paper_conf_ipps_luongmt10_b200 import _build
os.environ["LNS_LIB"] = os.environ.get("LNS_PROF_LIB") or _build.LIB_PROF
import numpy as np
import paper_conf_ipps_luongmt10_b200 as L, ppp_inputs as pi
names = ["A count+bins", "B rest (window consts, ps)", "C place+pieces", "D X build (rest)", "eval+reduce", "exchange",
         "apply: unrank", "B ballots+scans", "apply: bookkeeping", "C/D records (warp 0)", "-", "-"]
lib = L.load(build_if_missing=False)
fn = lib.lns_debug_phases; fn.restype = ctypes.c_int32; fn.argtypes = [ctypes.c_void_p]
for spec in sys.argv[1:] or ["C4:148:500"]:
    cfg, nb, iters = spec.split(":"); nb = int(nb); iters = int(iters)
    c = pi.CONFIGS[cfg]; inst = pi.config_instance(cfg)
    with L.Instance(inst.A, inst.S) as I:
        L.lns_config(I.ctx, nb)
        L.lns_tabu_run(I.ctx, c["k"], 20, -1, 3, None, 0)
        out = np.zeros(12, np.uint64); fn(out.ctypes.data)
        res = L.lns_tabu_run(I.ctx, c["k"], iters, -1, pi.config_seed(cfg), None, 0)
        ms = L.lns_last_kernel_ms(I.ctx)
        out = np.zeros(12, np.uint64); fn(out.ctypes.data)
        it = res["iters_done"]
        per = out.astype(np.float64) / (nb * it)
        print(f"{cfg} blocks={nb} iters={it} us/iter={ms*1e3/it:.2f} cycles/iter(sum phases)={per.sum():.0f}")
        for n_, v in zip(names, per):
            if v: print(f"   {n_:16s} {v:9.0f} cyc  {v/1.965e3:7.2f} us")
