"""examples/plan_and_solve.c: the C ABI used from plain C (gcc), the way a C
caller links libtds.so.  CPU: STATIC plans for B200 properties (SURVEY.md
§8(a) A1 values) and the canonical permutation (§8(c) item 5); GPU: a tuned
solve of a ragged batch with the residual checked on the host."""
import os
import subprocess

import pytest

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
PKG = os.path.join(ROOT, "paper_conf_ipps_davidsonzo11_b200")


@pytest.fixture(scope="module")
def exe(tmp_path_factory):
    if not os.path.exists(os.path.join(PKG, "libtds.so")):
        import __graft_entry__
        __graft_entry__.build()
    out = str(tmp_path_factory.mktemp("cex") / "plan_and_solve")
    cmd = ["gcc", "-std=c11", "-O2", "-Wall", "-Werror", os.path.join(ROOT, "examples", "plan_and_solve.c"),
           "-I" + os.path.join(ROOT, "include"), "-I/usr/local/cuda/include", "-L" + PKG, "-ltds",
           "-L/usr/local/cuda/lib64", "-lcudart", "-lm", "-Wl,-rpath," + PKG, "-o", out]
    subprocess.run(cmd, check=True, capture_output=True, text=True)
    return out


def _run(exe):
    r = subprocess.run([exe], capture_output=True, text=True, timeout=300)
    assert r.returncode == 0, r.stdout + r.stderr
    return r.stdout


def test_c_example_plans(exe):
    out = _run(exe)
    assert "STATIC n=1024 m=1: k=0 passes=0 n_sub=1024" in out
    assert "STATIC n=65536 m=256: k=3 passes=1 n_sub=8192" in out
    assert "STATIC n=1048576 m=16: k=7 passes=1 n_sub=8192" in out
    assert "STATIC n=16384 m=4096: k=1 passes=1 n_sub=8192" in out
    assert "permutation n=8 k=2: 0 4 1 5 2 6 3 7" in out


@pytest.mark.gpu
def test_c_example_solve(exe):
    out = _run(exe)
    assert "relative residual" in out and out.strip().endswith("ok"), out
