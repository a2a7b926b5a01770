"""The programmatic-dependent-launch discipline, checked in the built SASS (no
GPU needed; cuobjdump).

Every kernel launched with PDL may start while the previous kernel on the
stream still runs, so it must not touch global memory before its
griddepcontrol.wait (SASS ACQBULK): no global load, store, atomic or bulk copy
may precede the first ACQBULK (include/lift.h, csrc/common.cuh).  The only
memory instruction allowed there is the L2 bulk prefetch (UBLKPF.L2), which
delivers no data; the streaming kernels must issue it there (the prefetch of
their first bytes while the predecessor drains).
"""
import os
import re
import shutil
import subprocess

import pytest

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
LIB = os.path.join(ROOT, "paper_conf_cgo_steuwerrd17_b200", "liblift.so")

# global-memory instructions that may not run before the wait (CCTL.IVALL, the L1
# invalidate of a cluster barrier's acquire, touches no global data: allowed)
FORBIDDEN = re.compile(r"\b(LDG|STG|LD\.E|ST\.E|ATOMG|ATOM\.E|RED\.E|REDG|UBLKCP|UBLKRED|UTMALDG|UTMASTG|CCTL\.E)")


def sass_functions():
    exe = shutil.which("cuobjdump") or "/usr/local/cuda/bin/cuobjdump"
    if not os.path.exists(LIB):
        from paper_conf_cgo_steuwerrd17_b200 import build

        build.build()
    out = subprocess.run([exe, "-sass", LIB], capture_output=True, text=True, check=True).stdout
    funcs, name = {}, None
    for line in out.splitlines():
        m = re.search(r"Function : (\S+)", line)
        if m:
            name = m.group(1)
            funcs[name] = []
            continue
        if name is not None and re.search(r"/\*[0-9a-f]{4,}\*/", line):
            funcs[name].append(line)
    return funcs


@pytest.fixture(scope="module")
def funcs():
    return sass_functions()


def before_wait(lines):
    for i, line in enumerate(lines):
        if "ACQBULK" in line:
            return lines[:i]
    return None


def test_no_global_access_before_griddepcontrol_wait(funcs):
    checked = 0
    for name, lines in funcs.items():
        pre = before_wait(lines)
        if pre is None:
            continue
        checked += 1
        # the pattern does find this kernel's global accesses (after the wait)
        assert any(FORBIDDEN.search(line) for line in lines[len(pre):]), (name, "pattern matched nothing")
        bad = [line.strip() for line in pre if FORBIDDEN.search(line)]
        assert not bad, (name, bad[:3])
    assert checked >= 20, f"only {checked} kernels wait on their predecessor"


@pytest.mark.parametrize("pattern", [
    r"k_gemvILi1ELi4ELi8ELi1ELb1ELi4E",   # GEMV 4096^2 / 8192^2 (x in shared memory)
    r"k_gemvILi1ELi4ELi8ELi1ELb0ELi4E",   # the 8 GiB GEMV (x through L1)
    r"k_gemvILi2ELi4ELi8ELi1ELb1ELi4E",   # GESUMMV
    r"k_dotILi256ELi4ELb1E",              # dot (vector path)
    r"k_atax_fusedILi4ELi1E",             # fused ATAX 8192^2
    r"k_atax_fusedILi2ELi2E",             # fused ATAX 4096^2
    r"k_atax_colsILi4E",                  # two-pass column pass / transposed SGEMV
    r"k_listing1",                        # Listing-1 partialDot
    r"k_atax_fused_wideILi8E",            # wide-row fused ATAX
])
def test_streaming_kernels_prefetch_before_the_wait(funcs, pattern):
    hits = {k: v for k, v in funcs.items() if re.search(pattern, k)}
    assert hits, pattern
    for name, lines in hits.items():
        pre = before_wait(lines)
        assert pre is not None, (name, "no griddepcontrol.wait")
        assert any("UBLKPF.L2" in line for line in pre), (name, "no L2 prefetch before the wait")
