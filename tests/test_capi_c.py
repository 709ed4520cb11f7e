"""The boundary is a C ABI: include/vsched.h compiles as strict C11 (gcc -Werror) and a plain C
client linked against libvsched.so drives a SIM-mode tiled matmul through it (tests/c/capi_sim.c:
learning runs, first reliable decision, earliest-executor version choice; L428-475)."""
import os
import shutil
import subprocess

import pytest

import paper_conf_ipps_planasbal13_b200 as vs

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


@pytest.mark.skipif(shutil.which("gcc") is None, reason="gcc not available")
def test_plain_c_client_sim(tmp_path):
    lib = vs.lib()._name
    libdir = os.path.dirname(os.path.abspath(lib))
    exe = str(tmp_path / "capi_sim")
    cmd = ["gcc", "-std=c11", "-Wall", "-Wextra", "-Werror", "-I", os.path.join(ROOT, "include"),
           os.path.join(ROOT, "tests", "c", "capi_sim.c"), lib, "-Wl,-rpath," + libdir, "-o", exe]
    subprocess.run(cmd, check=True, capture_output=True, text=True)
    r = subprocess.run([exe], capture_output=True, text=True, timeout=120)
    assert r.returncode == 0, r.stderr
    assert "first reliable 5" in r.stdout
