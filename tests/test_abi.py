"""CPU-side checks of the C ABI boundary: the library builds for sm_100a, loads, and exports
every entry point include/lns.h declares; host-only entry points behave as documented."""
import os
import re
import subprocess

import pytest

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def _declared():
    src = open(os.path.join(ROOT, "include", "lns.h")).read()
    src = re.sub(r"/\*.*?\*/", "", src, flags=re.S)
    return sorted(set(re.findall(r"\b(lns_[a-z_]+)\s*\(", src)))


def test_header_declares_the_boundary_calls():
    names = _declared()
    for need in ("lns_create", "lns_eval_neighborhood", "lns_tabu_run", "lns_tabu_run_batch",
                 "lns_attach_comm", "lns_destroy", "lns_strerror", "lns_version", "lns_unrank"):
        assert need in names


def test_library_exports_every_declared_symbol():
    import paper_conf_ipps_luongmt10_b200 as L

    lib = L.load()
    out = subprocess.run(["nm", "-D", "--defined-only", L.library_path()], capture_output=True, text=True,
                         check=True).stdout
    exported = set(re.findall(r"\bT (lns_\w+)", out))
    for name in _declared():
        assert name in exported, name
        getattr(lib, name)
    assert set(L._SIGS) == set(_declared())


def test_library_is_sm100a():
    import paper_conf_ipps_luongmt10_b200 as L

    L.load()
    out = subprocess.run(["cuobjdump", "--list-elf", L.library_path()], capture_output=True, text=True).stdout
    assert "sm_100a" in out


def test_host_only_entry_points():
    import paper_conf_ipps_luongmt10_b200 as L
    from math import comb

    assert L.lns_version() >= 100
    for n in (1, 3, 21, 117, 1024, 2954):
        for k in (1, 2, 3):
            assert L.lns_neighborhood_size(n, k) == comb(n, k)
    for n, k in ((10, 4), (500, 4), (80, 7)):  # k > 3 (the generic-k path)
        assert L.lns_neighborhood_size(n, k) == comb(n, k)
    assert L.lns_neighborhood_size(10, 8) == -1
    assert L.lns_strerror(L.LNS_ENOADMISSIBLE) == "no admissible neighbour"
    cached, live = L.lns_pool_stats()  # host-only: the device-memory cache's counters
    assert cached >= 0 and live >= 0


def test_no_cpu_fallback_without_gpu():
    """On a host without a GPU the product path must fail loudly, never compute on the CPU."""
    import torch

    if torch.cuda.is_available():
        pytest.skip("GPU present")
    import numpy as np

    import paper_conf_ipps_luongmt10_b200 as L

    with pytest.raises(L.LnsError):
        L.lns_create(np.ones((2, 3), np.int8), np.array([3, 3], np.int32))


def _build_c_example(tmp_path):
    import os
    import shutil
    import subprocess

    import paper_conf_ipps_luongmt10_b200 as L

    cc = shutil.which("cc") or shutil.which("gcc")
    if not cc:
        pytest.skip("no C compiler")
    root = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
    libdir = os.path.dirname(L._build.LIB)
    L.load()  # builds liblns.so if missing
    exe = str(tmp_path / "tabu_c")
    subprocess.check_call([cc, "-O2", "-Wall", "-Werror", "-I", os.path.join(root, "include"),
                           os.path.join(root, "examples", "tabu_c.c"), "-L", libdir, "-llns",
                           f"-Wl,-rpath,{libdir}", "-o", exe])
    return exe


def test_c_example_builds_against_the_header_and_fails_loudly_without_gpu(tmp_path):
    """The boundary is a plain C ABI: examples/tabu_c.c (no Python, no torch) compiles against
    include/lns.h and links liblns.so; without a usable GPU its first call fails with a CUDA error
    (no CPU fallback)."""
    import subprocess

    import torch

    exe = _build_c_example(tmp_path)
    if torch.cuda.is_available():
        return
    out = subprocess.run([exe, "21", "21", "1", "10"], capture_output=True, text=True, timeout=120)
    assert out.returncode == 1 and "CUDA error" in out.stderr, out.stderr


def test_bench_refuses_more_gpus_than_visible():
    """bench.py --gpus N without torchrun re-launches itself with N ranks only if N GPUs are
    visible; otherwise it prints an error line and exits 2 (it never reports n_gpus: 1 for N > 1).
    On this GPU-less host: 0 visible GPUs."""
    import json
    import sys

    import torch

    if torch.cuda.is_available():
        pytest.skip("a GPU is visible")
    out = subprocess.run([sys.executable, os.path.join(ROOT, "bench.py"), "--gpus", "2", "--steps", "1"],
                         capture_output=True, text=True, timeout=300)
    assert out.returncode == 2, out.stdout + out.stderr
    line = json.loads(out.stdout.strip().splitlines()[-1])
    assert "error" in line and "--gpus 2" in line["error"]


def test_bench_reference_arm_ignores_gpu_count_on_nonzero_ranks():
    """--impl reference under torchrun: ranks other than 0 exit 0 without work (and print nothing)."""
    import sys

    env = {**os.environ, "RANK": "1", "WORLD_SIZE": "2", "LOCAL_RANK": "1"}
    out = subprocess.run([sys.executable, os.path.join(ROOT, "bench.py"), "--impl", "reference", "--gpus", "2"],
                         capture_output=True, text=True, timeout=300, env=env)
    assert out.returncode == 0 and out.stdout.strip() == "", out.stdout + out.stderr


def test_bench_context_lines_guard():
    """bench.py's context sections: an exception becomes {"error": ...} in its slot and
    the line is still printed; a section that never returns (a collective some rank did not reach)
    is cut by the watchdog, which prints the headline line and exits 0 instead of hanging."""
    import json
    import subprocess
    import sys

    root = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
    prog = (
        "import sys, time; sys.path.insert(0, %r); import bench\n"
        "line = {'metric': 'm', 'value': 1.0, 'a': None, 'b': None}\n"
        "c = bench.ContextLines(line, 0, %s)\n"
        "c.section('a', lambda: 1 / 0)\n"
        "c.section('b', lambda: {'ok': 1})\n"
        "%s\n"
        "c.finish()\n"
    )
    out = subprocess.run([sys.executable, "-c", prog % (root, "30", "")], capture_output=True, text=True, timeout=60)
    assert out.returncode == 0, out.stderr
    line = json.loads(out.stdout.strip().splitlines()[-1])
    assert line["value"] == 1.0 and "ZeroDivisionError" in line["a"]["error"] and line["b"] == {"ok": 1}
    assert "context_note" not in line
    hang = "c.section('c', lambda: time.sleep(60))"
    out = subprocess.run([sys.executable, "-c", prog % (root, "1", hang)], capture_output=True, text=True, timeout=60)
    assert out.returncode == 0, out.stderr
    line = json.loads(out.stdout.strip().splitlines()[-1])
    assert line["value"] == 1.0 and "stopped after 1 s" in line["context_note"] and "c" not in line
