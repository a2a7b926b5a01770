"""Launch-configuration sweep for the GEMV-family kernels (tuning aid).

Each configuration is timed as a CUDA graph of `reps` back-to-back calls over
rotating operand sets whose total exceeds L2 (so every call streams from HBM).
Prints us/call and GB/s (algorithmic bytes).
"""
import itertools
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import synth  # noqa: E402
import paper_conf_cgo_steuwerrd17_b200 as lift  # noqa: E402

dev = torch.device("cuda:0")


def graph_time(calls, reps=3):
    g = torch.cuda.CUDAGraph()
    for c in calls:
        c()
    torch.cuda.synchronize()
    with torch.cuda.graph(g):
        for c in calls:
            c()
    g.replay()
    torch.cuda.synchronize()
    best = 1e30
    for _ in range(reps):
        s, e = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        s.record()
        g.replay()
        e.record()
        e.synchronize()
        best = min(best, s.elapsed_time(e) * 1e3 / len(calls))
    return best


CONFIGS = [(8, 1), (8, 2), (4, 2), (4, 4), (2, 4), (2, 8), (1, 8)]
FULL = "--full" in sys.argv


def sweep(op, m, n, nsets, ncalls=24):
    sets = []
    for k in range(nsets):
        A = synth.torch_matrix_rows(2 + 10 * k, n, 0, m, device=dev)
        B = synth.torch_matrix_rows(3 + 10 * k, n, 0, m, device=dev) if op == "gesummv" else None
        sets.append((A, B))
    x = synth.torch_uniform(0, 0, n, device=dev)
    y = torch.empty(m, device=dev)
    nbytes = (8 if op == "gesummv" else 4) * m * n + 4 * (m + n)
    res = []

    def mk(A, B, **kw):
        if op == "gemv":
            return lambda: lift.lift_gemv_tuned(A, x, out=y, **kw)
        return lambda: lift.lift_gesummv_tuned(1.5, A, 1.2, B, x, out=y, **kw)

    auto = graph_time([(lambda A=A, B=B: (lift.lift_gemv(A, x, out=y) if op == "gemv" else
                                          lift.lift_gesummv(1.5, A, 1.2, B, x, out=y)))
                       for A, B in (sets * ncalls)[:ncalls]])
    print(f"{op} {m}x{n} auto: {auto:8.2f} us  {nbytes / auto / 1e3:7.1f} GB/s", flush=True)
    for (wpr, rg), xs, lb in (itertools.product(CONFIGS, (0, 1), (4, 8)) if FULL else ()):
        try:
            calls = [mk(A, B, wpr=wpr, rg=rg, xsmem=xs, lb=lb) for A, B in (sets * ncalls)[:ncalls]]
            t = graph_time(calls)
        except Exception as ex:  # unsupported combination
            print(f"  wpr={wpr} rg={rg} xs={xs} lb={lb}: {str(ex)[:60]}")
            continue
        res.append((t, wpr, rg, xs, lb))
        print(f"  wpr={wpr} rg={rg} xs={xs} lb={lb}: {t:8.2f} us  {nbytes / t / 1e3:7.1f} GB/s", flush=True)
    if "--blocks-fine" in sys.argv:  # grid sizes around the row count's divisors x configs
        grid = [(wpr, rg, blocks) for wpr, rg in ((8, 1), (4, 2), (2, 4), (8, 2), (4, 4))
                for blocks in (256, 296, 341, 384, 444, 512, 592, 683, 740, 768, 888, 1024, 1184)]
        xss = (1,)
    else:
        grid = [(8, 1, blocks) for blocks in (296, 444, 592, 888, 1184, 1776, 2368)]
        xss = (0, 1)
    for wpr, rg, blocks in grid:
        for xs in xss:
            calls = [mk(A, B, wpr=wpr, rg=rg, xsmem=xs, lb=4, blocks=blocks) for A, B in (sets * ncalls)[:ncalls]]
            t = graph_time(calls)
            res.append((t, wpr, rg, xs, 4, blocks))
            print(f"  wpr={wpr} rg={rg} xs={xs} lb=4 blocks={blocks}: {t:8.2f} us  {nbytes / t / 1e3:7.1f} GB/s",
                  flush=True)
    res.sort()
    print(f"BEST {op} {m}x{n}: {res[0]}", flush=True)
    del sets
    torch.cuda.empty_cache()


if __name__ == "__main__":
    which = [a for a in sys.argv[1:] if not a.startswith("--")] or ["gemv4096", "gemv8192", "gesummv8192", "gemv65536"]
    if "gemv4096" in which:
        sweep("gemv", 4096, 4096, nsets=6)
    if "gemv8192" in which:
        sweep("gemv", 8192, 8192, nsets=2)
    if "gesummv8192" in which:
        sweep("gesummv", 8192, 8192, nsets=1)
    if "gesummv4096" in which:
        sweep("gesummv", 4096, 4096, nsets=3)
    if "gemv65536" in which:
        sweep("gemv", 65536, 32768, nsets=1, ncalls=4)
