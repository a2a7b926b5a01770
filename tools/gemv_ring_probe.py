"""Experiment: would a bulk-copy-ring GEMV (one block per SM, the fused ATAX's
stage ring and per-row block reduction, t_r written out instead of the rank-1
updates) beat k_gemv?  Needs LIFT_ROOT at a tree built with
-DLIFT_EXP_GEMV_RING (lift_atax then returns A x).  Prints both, back to back
(graphs of 32 calls, operands rotated past L2, median of 5) and checks the ring
result against lift_gemv within the tolerance.
usage: LIFT_ROOT=<exp tree> python tools/gemv_ring_probe.py"""
import os
import statistics
import sys

import torch

sys.path.insert(0, os.environ["LIFT_ROOT"])
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
    return statistics.median(per)


for n in (4096, 8192):
    copies = max(2, -(-3 * L2 // (4 * n * n)))
    As = [synth.torch_matrix_rows(2 + k, n, 0, n, device=dev) for k in range(copies)]
    x = synth.torch_uniform(0, 0, n, device=dev)
    y1, y2 = torch.empty(n, device=dev), torch.empty(n, device=dev)
    lift.lift_gemv(As[0], x, out=y1)
    lift.lift_atax(As[0], x, out=y2, algo="fused")
    torch.cuda.synchronize()
    err = ((y1 - y2).abs().max() / y1.abs().max()).item()
    for rep in range(3):
        tg = timeit([(lambda A=A: lift.lift_gemv(A, x, out=y1)) for A in As])
        tr = timeit([(lambda A=A: lift.lift_atax(A, x, out=y2, algo="fused")) for A in As])
        print(f"{n}^2: k_gemv {tg:7.2f} us   ring GEMV {tr:7.2f} us   (rel. diff {err:.1e})", flush=True)
    del As
