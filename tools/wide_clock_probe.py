"""Is the wide-row ATAX sensitive to the clock state a long HBM stream leaves?
Times 8192x32768 fused ATAX fresh, right after ~3 s of back-to-back 2^28 dots,
and again after 2 s idle; samples the SM clock with nvidia-smi each time.
usage: python tools/wide_clock_probe.py"""
import os
import subprocess
import sys
import time

import torch

sys.path.insert(0, os.getcwd())
sys.path.insert(0, os.path.join(os.getcwd(), "tools"))
import synth  # noqa: E402
import paper_conf_cgo_steuwerrd17_b200 as lift  # noqa: E402
from sweep import graph_time  # noqa: E402

dev = torch.device("cuda:0")
m, n = 8192, 32768
x = synth.torch_uniform(0, 0, n, device=dev)
y = torch.empty(n, device=dev)
As = [synth.torch_matrix_rows(2 + 10 * k, n, 0, m, device=dev) for k in range(2)]
calls = [(lambda A=A: lift.lift_atax(A, x, out=y, algo="fused")) for A in (As * 12)[:12]]
dx = synth.torch_uniform(5, 0, 1 << 28, device=dev)
dy = synth.torch_uniform(6, 0, 1 << 28, device=dev)
r = torch.empty((), device=dev)


def clock():
    return subprocess.run(["nvidia-smi", "--query-gpu=clocks.sm,power.draw", "--format=csv,noheader"],
                          capture_output=True, text=True).stdout.strip()


print("fresh          ", f"{graph_time(calls):8.2f} us", clock(), flush=True)
t0 = time.time()
while time.time() - t0 < 3:
    for _ in range(50):
        lift.lift_dot(dx, dy, out=r)
    torch.cuda.synchronize()
print("after dot load ", f"{graph_time(calls):8.2f} us", clock(), flush=True)
time.sleep(2)
print("after 2 s idle ", f"{graph_time(calls):8.2f} us", clock(), flush=True)
