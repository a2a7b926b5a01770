"""Why do the bench's Table-1 timings of the small ops read higher than its ops
block?  Times GEMV 4096^2 / ATAX 4096^2 in one process, alternating, with the
operand layouts of both blocks: (a) separate clones of A (the ops block), (b)
slices of one large pool with x at the pool's tail (bench.table1_calls), and
(c) pool slices with a separate x.  Graphs of 32 back-to-back calls, median /
min of 5 replays.
usage: python tools/table1_vs_ops_probe.py"""
import os
import statistics
import sys

import torch

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import synth  # noqa: E402
import paper_conf_cgo_steuwerrd17_b200 as lift  # noqa: E402

dev = torch.device("cuda:0")
L2 = torch.cuda.get_device_properties(dev).L2_cache_size


def timeit(calls, reps=32):
    seq = [calls[j % len(calls)] for j in range(reps)]
    for c in calls:
        c()
    g = torch.cuda.CUDAGraph()
    with torch.cuda.graph(g):
        for c in seq:
            c()
    g.replay()
    torch.cuda.synchronize()
    per = []
    for _ in range(5):
        s, e = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        s.record()
        g.replay()
        e.record()
        e.synchronize()
        per.append(s.elapsed_time(e) * 1e3 / reps)
    return statistics.median(per), min(per)


pool = synth.torch_uniform(synth.SEED_A, 0, (8 << 30) // 4, device=dev)  # 8 GiB, like the bench's GEMV A
for op, m, n in (("gemv", 4096, 4096), ("atax", 4096, 4096)):
    per = m * n
    copies = int(-(-2 * L2 // (4 * per))) + 1
    clones = [synth.torch_matrix_rows(2 + 10 * k, n, 0, m, device=dev) for k in range(copies)]
    slices = [pool[k * per:(k + 1) * per].view(m, n) for k in range(copies)]
    x_tail = pool[-n:]
    x_sep = synth.torch_uniform(0, 0, n, device=dev)
    y = torch.empty(m if op == "gemv" else n, device=dev)
    f = (lambda A, x: lift.lift_gemv(A, x, out=y)) if op == "gemv" else (lambda A, x: lift.lift_atax(A, x, out=y))
    for rep in range(3):
        for label, As, x in (("clones, own x", clones, x_sep), ("pool slices, x at pool tail", slices, x_tail),
                             ("pool slices, own x", slices, x_sep), ("clones, x at pool tail", clones, x_tail)):
            med, mn = timeit([(lambda A=A: f(A, x)) for A in As])
            print(f"{op} {m}x{n} {label:30s} median {med:6.2f} us  min {mn:6.2f}", flush=True)
    del clones
