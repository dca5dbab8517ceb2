import sys, os, ctypes
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import paper_conf_ipps_luongmt10_b200 as L, ppp_inputs as pi
inst = pi.config_instance("C5"); n = 1024; k = int(sys.argv[1])
V = pi.start_vector(n, pi.config_seed("C5"))
ctx = L.lns_create(inst.A, inst.S)
lib = L.load()
fn = lib.lns_debug_plan; fn.restype = ctypes.c_int32
fn.argtypes = [ctypes.c_void_p, ctypes.c_int32, ctypes.c_void_p, ctypes.c_void_p, ctypes.c_int64]
out = np.zeros(8000, np.int32)
print(fn(ctx, k, V.ctypes.data, out.ctypes.data, 8000))
np.save(f"gpurun_out/plan_k{k}.npy", out)
