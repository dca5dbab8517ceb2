"""Time the parts of the bench's end-to-end leg: lns_create (host A/S), the batched job, lns_destroy."""
import os, sys, time
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np, torch
import paper_conf_ipps_luongmt10_b200 as L, ppp_inputs as pi
inst = pi.config_instance("C4")
A_h = torch.from_numpy(inst.A).pin_memory(); S_h = torch.from_numpy(inst.S).pin_memory()
V0 = torch.from_numpy(np.stack([pi.start_vector(inst.n, pi.restart_seed(5, r)) for r in range(50)])).pin_memory()
Vo = torch.empty((50, inst.n), dtype=torch.int8).pin_memory()
torch.cuda.init(); torch.cuda.synchronize()
for rep in range(4):
    t0 = time.perf_counter(); c = L.lns_create(A_h, S_h, 0); torch.cuda.synchronize(); t1 = time.perf_counter()
    r = L.lns_tabu_run_batch(c, 3, 50, 400, -1, 0, V0, 0, Vo, torch.cuda.current_stream()); torch.cuda.synchronize(); t2 = time.perf_counter()
    km = L.lns_last_kernel_ms(c)
    L.lns_destroy(c); torch.cuda.synchronize(); t3 = time.perf_counter()
    print(f"create {1e3*(t1-t0):.2f} ms  batch {1e3*(t2-t1):.2f} ms (kernel {km:.2f})  destroy {1e3*(t3-t2):.2f} ms")

# the bench's loop: events on the stream around create + batch + destroy, after an L2 flush
main = L.lns_create(torch.from_numpy(inst.A).cuda(), torch.from_numpy(inst.S).cuda(), 0)
L.lns_tabu_run_batch(main, 3, 50, 400, -1, 0, V0.cuda(), 0, Vo.cuda(), torch.cuda.current_stream())
flush = torch.empty(512 * 2**20 // 4, dtype=torch.int32, device="cuda")
st = torch.cuda.current_stream()
for i in range(4):
    flush.fill_(i); torch.cuda.synchronize()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    e0.record(st); t0 = time.perf_counter()
    c2 = L.lns_create(A_h, S_h, 0)
    r2 = L.lns_tabu_run_batch(c2, 3, 50, 400, -1, 0, V0, 0, Vo, st)
    km = L.lns_last_kernel_ms(c2)
    L.lns_destroy(c2)
    e1.record(st); torch.cuda.synchronize()
    print(f"bench-style e2e: events {e0.elapsed_time(e1):.2f} ms, host {1e3*(time.perf_counter()-t0):.2f} ms, kernel {km:.2f} ms")
