"""Write tests/golden/c5_trajectory.txt: the first iterations of the C5 tabu search, computed by
the CPU ORACLE ONLY (oracle/ + the seeded generators of ppp_inputs; nothing from the CUDA path).

C5 = BASELINE.json configs[4]: planted 1024 x 1024 instance (instance seed 1005), 3-Hamming
neighbourhood (C(1024,3) = 178,433,024 neighbours, PAPER.md:119-125 / Fig. 10), run
seed 6, tenure floor(M/6), no early stop. Each iteration is the tabu iteration of
PAPER.md:241-258 (Section IV-B): every neighbour's fitness from scratch, lowest rank
wins ties (reading R5). About 20 min per iteration on 8 host cores.

    python scripts/golden_c5.py [iters]
"""
import hashlib
import os
import sys
import time

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import numpy as np  # noqa: E402

import oracle  # noqa: E402
import ppp_inputs as pi  # noqa: E402

OUT = os.path.join(ROOT, "tests", "golden", "c5_trajectory.txt")


def main(iters: int) -> None:
    inst = pi.config_instance("C5")
    seed = pi.config_seed("C5")
    V0 = pi.start_vector(inst.n, seed)
    ten = pi.default_tenure(inst.n, 3)
    t0 = time.time()
    tr, tf, Vo, res = oracle.tabu_run(inst.A, inst.S, 3, V0, iters, ten, stop_on_zero=False)
    dt = time.time() - t0
    f0 = oracle.fitness(inst.A, inst.S, V0, packed=True)
    vh = hashlib.sha256(np.ascontiguousarray(Vo, dtype=np.int8).tobytes()).hexdigest()
    with open(OUT, "w") as fh:
        fh.write("# C5 tabu trajectory, written by scripts/golden_c5.py from oracle/ only.\n")
        fh.write("# BASELINE.json configs[4]: planted 1024x1024 (instance seed 1005), k = 3, run seed 6,\n")
        fh.write(f"# tenure {ten} = floor(C(1024,3)/6) (PAPER.md:253-255), no early stop; tabu iteration of\n")
        fh.write("# PAPER.md:241-258 (Section IV-B), fitness P:231-237, lowest rank wins ties (DESIGN R5).\n")
        fh.write(f"# oracle wall time {dt:.0f} s on {oracle.max_threads()} threads\n")
        fh.write(f"f0 {f0}\n")
        for t in range(len(tr)):
            fh.write(f"{t + 1} {int(tr[t])} {int(tf[t])}\n")
        fh.write(f"V_out_sha256 {vh}\n")
        fh.write("result " + " ".join(f"{k}={v}" for k, v in res.items()) + "\n")
    print(open(OUT).read())


if __name__ == "__main__":
    main(int(sys.argv[1]) if len(sys.argv) > 1 else 3)
