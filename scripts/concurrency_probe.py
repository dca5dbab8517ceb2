"""Do two persistent (cooperative) searches on two streams of one GPU run concurrently?"""
import os, sys, threading, time
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np, torch
import paper_conf_ipps_luongmt10_b200 as L, ppp_inputs as pi
inst = pi.config_instance("C4"); V0 = pi.start_vector(inst.n, 3)
mode = sys.argv[2] if len(sys.argv) > 2 else "host"
if mode == "device":
    V0 = torch.from_numpy(V0).cuda()
elif mode == "pinned":
    V0 = torch.from_numpy(V0).pin_memory()
ctxs = [L.lns_create(inst.A, inst.S) for _ in range(2)]
for c in ctxs:
    L.lns_config(c, int(sys.argv[1]) if len(sys.argv) > 1 else 32)
    L.lns_tabu_run(c, 3, 300, -1, 0, V0, 0)
streams = [torch.cuda.Stream() for _ in ctxs]
t_single = time.perf_counter(); L.lns_tabu_run(ctxs[0], 3, 300, -1, 0, V0, 0, stream=streams[0]); t_single = time.perf_counter() - t_single
marks = {}
def run(p):
    marks[(p, 's')] = time.perf_counter()
    L.lns_tabu_run(ctxs[p], 3, 300, -1, 0, V0, 0, stream=streams[p])
    marks[(p, 'e')] = time.perf_counter()
t0 = time.perf_counter()
th = [threading.Thread(target=run, args=(p,)) for p in range(2)]
[t.start() for t in th]; [t.join() for t in th]
tot = time.perf_counter() - t0
print(f"[{mode}] single {t_single*1e3:.1f} ms; two threads {tot*1e3:.1f} ms (overlap if ~single, serial if ~2x)")
print("kernel ms", [round(L.lns_last_kernel_ms(c), 2) for c in ctxs])
for p in range(2):
    print(p, f"start {1e3*(marks[(p,'s')]-t0):.1f} end {1e3*(marks[(p,'e')]-t0):.1f}")
