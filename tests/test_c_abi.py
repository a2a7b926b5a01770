"""The C ABI from a plain C11 program (tests/c/abi_consumer.c): no Python
between the caller and liblift.so.  CPU: it compiles with -Wall -Werror
against include/*.h, links, and gets the documented status codes; GPU: every
entry point it calls matches the fp64 oracle within the north_star
tolerance."""
import os
import subprocess

import pytest

import oracle
import paper_conf_cgo_steuwerrd17_b200 as lift

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
CUDA = os.environ.get("CUDA_HOME", "/usr/local/cuda")


@pytest.fixture(scope="module")
def consumer(tmp_path_factory):
    libdir = os.path.dirname(lift.library_path())
    odir = os.path.dirname(oracle.build())
    exe = str(tmp_path_factory.mktemp("cabi") / "abi_consumer")
    cmd = ["gcc", "-std=c11", "-O2", "-Wall", "-Wextra", "-Werror", "-I", os.path.join(ROOT, "include"),
           "-I", os.path.join(ROOT, "oracle"), "-I", os.path.join(CUDA, "include"),
           os.path.join(ROOT, "tests", "c", "abi_consumer.c"), "-o", exe,
           "-L", libdir, "-llift", "-L", odir, "-loracle", "-L", os.path.join(CUDA, "lib64"), "-lcudart", "-lm",
           f"-Wl,-rpath,{libdir}:{odir}:{os.path.join(CUDA, 'lib64')}"]
    r = subprocess.run(cmd, capture_output=True, text=True)
    assert r.returncode == 0, r.stderr
    return exe


def test_c_consumer_builds_and_status_codes(consumer):
    r = subprocess.run([consumer, "--no-gpu"], capture_output=True, text=True, timeout=120)
    assert r.returncode == 0, r.stdout + r.stderr
    assert "ABI OK" in r.stdout


@pytest.mark.gpu
def test_c_consumer_parity_gpu(consumer, cuda_device):
    r = subprocess.run([consumer], capture_output=True, text=True, timeout=600)
    assert r.returncode == 0, r.stdout + r.stderr
    assert "ABI OK" in r.stdout and r.stdout.count("margin") >= 12
