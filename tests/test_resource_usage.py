"""Register / stack budgets of the hot kernels, read from the built library
with cuobjdump (no GPU needed).  The launch shapes the B200 sweeps picked
rely on them: k_gemv's 256-thread blocks run 4 per SM only at <= 64
registers, and no hot kernel may spill (a stack frame means local-memory
traffic inside the stream)."""
import os
import re
import shutil
import subprocess

import pytest

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
LIB = os.path.join(ROOT, "paper_conf_cgo_steuwerrd17_b200", "liblift.so")


def usage():
    exe = shutil.which("cuobjdump") or "/usr/local/cuda/bin/cuobjdump"
    if not os.path.exists(LIB):
        from paper_conf_cgo_steuwerrd17_b200 import build

        build.build()
    out = subprocess.run([exe, "-res-usage", LIB], capture_output=True, text=True, check=True).stdout
    res, name = {}, None
    for line in out.splitlines():
        m = re.search(r"Function (\S+):", line)
        if m:
            name = m.group(1)
            continue
        m = re.search(r"REG:(\d+) STACK:(\d+)", line)
        if m and name:
            res[name] = (int(m.group(1)), int(m.group(2)))
    return res


@pytest.fixture(scope="module")
def res():
    return usage()


def pick(res, pattern):
    hits = {k: v for k, v in res.items() if re.search(pattern, k)}
    assert hits, pattern
    return hits


def test_gemv_default_shapes_fit_four_blocks_per_sm(res):
    # k_gemv<NMAT, 4, 8, 1, XSMEM, 4>: the automatic launch of the configs' shapes — GEMV
    # with x in shared memory (4096^2, 8192^2) or through L1 (65536 x 32768), GESUMMV with
    # x in shared memory (4096^2, 8192^2)
    for pat in (r"k_gemvILi1ELi4ELi8ELi1ELb[01]ELi4EEE", r"k_gemvILi2ELi4ELi8ELi1ELb1ELi4EEE"):
        for k, (reg, stack) in pick(res, pat).items():
            assert reg <= 64 and stack == 0, (k, reg, stack)


def test_hot_kernels_do_not_spill(res):
    for pat in (r"k_dotILi256ELi4ELb1E", r"k_atax_fusedILi[124]ELi[124]E", r"k_atax_fused_wideILi8E",
                r"k_listing1", r"k_atax_colsILi4E"):
        for k, (reg, stack) in pick(res, pat).items():
            assert stack == 0, (k, reg, stack)
