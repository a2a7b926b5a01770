"""Where does the fixed per-kernel cost come from?  (tuning aid)"""
import sys
import os

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import synth  # noqa: E402
import paper_conf_cgo_steuwerrd17_b200 as lift  # noqa: E402

dev = torch.device("cuda:0")
ev = lambda: torch.cuda.Event(enable_timing=True)  # noqa: E731


def loop_time(fn, reps=50, flush=None):
    """average per-call device time of `reps` back-to-back calls (one event pair)"""
    fn()
    torch.cuda.synchronize()
    if flush is not None:
        flush.sum()
    s, e = ev(), ev()
    s.record()
    for _ in range(reps):
        fn()
    e.record()
    e.synchronize()
    return s.elapsed_time(e) * 1e3 / reps


def graph_time(fn, reps=50):
    g = torch.cuda.CUDAGraph()
    fn()
    torch.cuda.synchronize()
    with torch.cuda.graph(g):
        for _ in range(reps):
            fn()
    g.replay()
    torch.cuda.synchronize()
    s, e = ev(), ev()
    s.record()
    g.replay()
    e.record()
    e.synchronize()
    return s.elapsed_time(e) * 1e3 / reps


def single(fn, flush):
    ts = []
    for _ in range(10):
        flush.sum()
        s, e = ev(), ev()
        s.record()
        fn()
        e.record()
        e.synchronize()
        ts.append(s.elapsed_time(e) * 1e3)
    ts.sort()
    return ts[5]


flush = torch.ones(128 << 20, device=dev)
for n in (4, 1 << 16, 1 << 20, 1 << 22, 1 << 24):
    x = synth.torch_uniform(0, 0, n, device=dev)
    y = synth.torch_uniform(1, 0, n, device=dev)
    f = lambda: lift.lift_dot(x, y)  # noqa: E731
    print(f"dot n={n:>9}: single(flushed) {single(f, flush):8.2f} us   loop(L2-warm) {loop_time(f):8.2f} us   graph {graph_time(f):8.2f} us", flush=True)
for m, n in ((256, 4096), (1024, 4096), (4096, 4096), (8192, 8192)):
    A = synth.torch_matrix_rows(2, n, 0, m, device=dev)
    x = synth.torch_uniform(0, 0, n, device=dev)
    yv = torch.empty(m, device=dev)
    f = lambda: lift.lift_gemv(A, x, out=yv)  # noqa: E731
    print(f"gemv {m}x{n}: single(flushed) {single(f, flush):8.2f} us   loop(L2-warm) {loop_time(f):8.2f} us   graph {graph_time(f):8.2f} us", flush=True)
# rotating buffers bigger than L2 (no flush kernel at all)
m, n = 4096, 4096
As = [synth.torch_matrix_rows(2 + k, n, 0, m, device=dev) for k in range(8)]  # 512 MiB total
x = synth.torch_uniform(0, 0, n, device=dev)
yv = torch.empty(m, device=dev)
k = [0]


def rot():
    lift.lift_gemv(As[k[0] % 8], x, out=yv)
    k[0] += 1


print(f"gemv 4096x4096 rotating 8 buffers: loop {loop_time(rot, reps=64):8.2f} us  graph {graph_time(rot, reps=64):8.2f} us")
xs = [synth.torch_uniform(10 + j, 0, 1 << 20, device=dev) for j in range(64)]
j = [0]


def rotd():
    lift.lift_dot(xs[j[0] % 64], xs[(j[0] + 1) % 64])
    j[0] += 1


print(f"dot 2^20 rotating 64 buffers (256 MiB): loop {loop_time(rotd, reps=64):8.2f} us  graph {graph_time(rotd, reps=64):8.2f} us")
