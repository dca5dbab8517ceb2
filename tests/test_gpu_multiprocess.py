"""The multi-process product path on ONE GPU (every gpurun box has one): two processes, each with
its own context on cuda:0, run the partitioned search of PAPER.md:448-454 ("partitioning the
neighborhood set, where each partition is executed on a single GPU") through the real library:

* ``stepped``: a gloo process group + the real ``LnsStepper`` (lns_step_eval / lns_step_apply of
  liblns.so) + ``parallel.partitioned_tabu_run`` (one all-reduce MIN of the int64 key per
  iteration);
* ``peer``: ``parallel.peer_tabu_run`` -- the device-initiated exchange with the exchange buffers
  shared as CUDA IPC handles across the two processes (cudaIpcOpenMemHandle, red.min.sys /
  red.release.sys / ld.acquire.sys), persistent kernels launched plainly (LNS_PLAIN_LAUNCH). The
  two contexts time-slice on the one device, so every exchange waits for a context switch: few
  iterations, generous timeout.

Both ranks must reproduce the ORACLE's single-process trajectory bit for bit.
"""
import os
import socket

import numpy as np
import pytest

import ppp_inputs as pi

pytestmark = pytest.mark.gpu


def _free_port():
    with socket.socket() as s:
        s.bind(("127.0.0.1", 0))
        return s.getsockname()[1]


def _worker(rank, world, port, cfg, iters, mode, outdir):
    import torch
    import torch.distributed as dist

    os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        torch.cuda.set_device(0)
        import paper_conf_ipps_luongmt10_b200 as L
        from paper_conf_ipps_luongmt10_b200 import parallel as par

        c = pi.CONFIGS[cfg]
        inst = pi.config_instance(cfg)
        k, n = c["k"], inst.n
        V0 = pi.start_vector(n, pi.config_seed(cfg))
        ctx = L.lns_create(inst.A, inst.S, 0)
        try:
            if mode == "stepped":
                st = par.LnsStepper(ctx, n, k, iters, -1, 0, V0, stop_on_zero=False, rank=rank, world=world)
                tr, tf, Vo, res = par.partitioned_tabu_run(st, iters)
            else:
                tr, tf = np.zeros(iters, np.int64), np.zeros(iters, np.int64)
                Vo = np.zeros(n, np.int8)
                res = par.peer_tabu_run(ctx, k, iters, -1, 0, V0, L.LNS_PLAIN_LAUNCH, timeout_ms=60000,
                                        V_out=Vo, trace_rank=tr, trace_fit=tf)
        finally:
            L.lns_destroy(ctx)
        np.savez(os.path.join(outdir, f"r{rank}.npz"), tr=np.asarray(tr), tf=np.asarray(tf), Vo=Vo,
                 res=np.array([res[f] for f in L.RESULT_FIELDS], np.int64))
    finally:
        dist.destroy_process_group()


@pytest.mark.parametrize("mode,cfg,iters", [("stepped", "C3", 60), ("stepped", "C4", 30), ("peer", "C2", 24),
                                            ("peer", "C3", 12)])
def test_two_processes_partitioned_search(orc, tmp_path, mode, cfg, iters):
    import torch

    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    import torch.multiprocessing as mp

    import paper_conf_ipps_luongmt10_b200 as L

    L.load()  # build in the parent: the children only load the library
    c = pi.CONFIGS[cfg]
    inst = pi.config_instance(cfg)
    V0 = pi.start_vector(inst.n, pi.config_seed(cfg))
    otr, otf, oVo, ores = orc.tabu_run(inst.A, inst.S, c["k"], V0, iters, pi.default_tenure(inst.n, c["k"]),
                                       stop_on_zero=False)
    mp.spawn(_worker, args=(2, _free_port(), cfg, iters, mode, str(tmp_path)), nprocs=2, join=True)
    for rank in range(2):
        got = np.load(tmp_path / f"r{rank}.npz")
        assert np.array_equal(got["tr"], otr), (rank, got["tr"][:8], otr[:8])
        assert np.array_equal(got["tf"], otf)
        assert np.array_equal(got["Vo"], oVo)
        assert list(got["res"]) == [ores[f] for f in L.RESULT_FIELDS]
