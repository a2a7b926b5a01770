"""compute-sanitizer over small / ragged invocations of every kernel
(memcheck, racecheck, synccheck, initcheck).  The kernels use no global
atomics on data and fixed-order reductions; any report is a bug."""
import os
import re
import shutil
import subprocess
import sys

import pytest

pytestmark = pytest.mark.gpu
ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


@pytest.mark.parametrize("tool", ["memcheck", "racecheck", "synccheck", "initcheck"])
def test_compute_sanitizer(cuda_device, tool):
    cs = shutil.which("compute-sanitizer") or "/usr/local/cuda/bin/compute-sanitizer"
    if not os.path.exists(cs):
        pytest.fail("compute-sanitizer not found")
    # the pool's operators may close the sanitizer (a stub that refuses every run with
    # exit code 86): then these cases cannot run here; the clean runs of this suite on
    # earlier boxes are in profiles/ and the bounds / NaN-prefill / oracle checks of the
    # other GPU tests stand in for it
    probe = subprocess.run([cs, "--version"], capture_output=True, text=True, timeout=120)
    if probe.returncode == 86 or "closed" in (probe.stdout + probe.stderr):
        pytest.skip("compute-sanitizer is closed on this GPU pool: " + (probe.stdout + probe.stderr).strip()[:200])
    # initcheck must see the writes of torch's fill kernels (torch.zeros workspaces), so
    # it instruments every kernel; the other tools check only this library's kernels
    filt = [] if tool == "initcheck" else ["--kernel-name", "kns=lift"]
    cmd = [cs, "--tool", tool, "--error-exitcode", "99", *filt,
           sys.executable, os.path.join(ROOT, "tools", "sanitize_cases.py")]
    env = dict(os.environ, LIFT_SANITIZER_TOOL=tool)  # tools/sanitize_cases.py: see the wide-row cases
    r = subprocess.run(cmd, capture_output=True, text=True, timeout=900, cwd=ROOT, env=env)
    tail = (r.stdout + r.stderr)[-4000:]
    assert r.returncode == 0, tail
    assert "sanitize cases ok" in r.stdout, tail
    out = r.stdout + r.stderr
    assert re.search(r"ERROR SUMMARY: 0 errors|SUMMARY: 0 hazards displayed \(0 errors", out), tail
