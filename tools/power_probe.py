"""Does a long run of the 2^31 dot slow down under the power cap?

Times graphs of K back-to-back dot launches (K = 1, 4, 16, 64) and samples
NVML SM / memory clocks, power and throttle reasons while they run.
usage: python tools/power_probe.py
"""
import os
import statistics
import sys
import threading
import time

import pynvml
import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import synth  # noqa: E402
import paper_conf_cgo_steuwerrd17_b200 as lift  # noqa: E402

dev = torch.device("cuda:0")
n = 1 << 31
x = synth.torch_uniform(0, 0, n, device=dev)
y = synth.torch_uniform(1, 0, n, device=dev)
out = torch.empty((), device=dev)
pynvml.nvmlInit()
h = pynvml.nvmlDeviceGetHandleByIndex(0)


def sample(stop, rec):
    while not stop.is_set():
        rec.append((pynvml.nvmlDeviceGetClockInfo(h, pynvml.NVML_CLOCK_SM),
                    pynvml.nvmlDeviceGetClockInfo(h, pynvml.NVML_CLOCK_MEM),
                    pynvml.nvmlDeviceGetPowerUsage(h) / 1000.0,
                    pynvml.nvmlDeviceGetCurrentClocksEventReasons(h)))
        time.sleep(0.002)


for K in (1, 4, 16, 64):
    lift.lift_dot(x, y, out=out)
    torch.cuda.synchronize()
    g = torch.cuda.CUDAGraph()
    with torch.cuda.graph(g):
        for _ in range(K):
            lift.lift_dot(x, y, out=out)
    g.replay()
    torch.cuda.synchronize()
    time.sleep(1.0)  # cool down
    rec, stop = [], threading.Event()
    t = threading.Thread(target=sample, args=(stop, rec))
    t.start()
    time.sleep(0.01)
    a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    a.record()
    g.replay()
    b.record()
    b.synchronize()
    stop.set()
    t.join()
    ms = a.elapsed_time(b) / K
    busy = rec[2:] if len(rec) > 4 else rec
    reasons = 0
    for r in busy:
        reasons |= r[3]
    print(f"dot 2^31 x{K:3d}: {ms * 1e3:8.1f} us/launch  {(8 * n + 4) / ms / 1e6:7.1f} GB/s  "
          f"sm {statistics.median(r[0] for r in busy):.0f} MHz  mem {statistics.median(r[1] for r in busy):.0f} MHz  "
          f"power max {max(r[2] for r in busy):.0f} W  reasons 0x{reasons:x}  samples {len(busy)}", flush=True)
