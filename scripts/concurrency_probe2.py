"""Does a torch kernel on stream B overlap lns_tabu_run on stream A? And two lns runs launched
from ONE thread (first call returns only after its sync, so use two contexts sequentially issued)?"""
import os, sys, threading, time
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np, torch
import paper_conf_ipps_luongmt10_b200 as L, ppp_inputs as pi
inst = pi.config_instance("C4"); V0 = torch.from_numpy(pi.start_vector(inst.n, 3)).cuda()
c = L.lns_create(inst.A, inst.S); L.lns_config(c, 32); L.lns_tabu_run(c, 3, 300, -1, 0, V0, 0)
sa, sb = torch.cuda.Stream(), torch.cuda.Stream()
# calibrate a ~8 ms sleep
with torch.cuda.stream(sb):
    torch.cuda._sleep(1000000); torch.cuda.synchronize()
    t = time.perf_counter(); torch.cuda._sleep(15000000); torch.cuda.synchronize(); print(f"sleep alone {1e3*(time.perf_counter()-t):.1f} ms")
t = time.perf_counter(); L.lns_tabu_run(c, 3, 300, -1, 0, V0, 0, stream=sa); print(f"lns alone {1e3*(time.perf_counter()-t):.1f} ms")
def other():
    with torch.cuda.stream(sb):
        torch.cuda._sleep(15000000)
    sb.synchronize()
t = time.perf_counter()
th = threading.Thread(target=other); th.start()
L.lns_tabu_run(c, 3, 300, -1, 0, V0, 0, stream=sa)
th.join()
print(f"lns + sleep (threads) {1e3*(time.perf_counter()-t):.1f} ms")
# same thread: sleep first (async), then lns (blocking)
t = time.perf_counter()
with torch.cuda.stream(sb):
    torch.cuda._sleep(15000000)
L.lns_tabu_run(c, 3, 300, -1, 0, V0, 0, stream=sa)
torch.cuda.synchronize()
print(f"sleep then lns (one thread) {1e3*(time.perf_counter()-t):.1f} ms")
