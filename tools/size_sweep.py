"""Achieved GB/s against bytes per launch for every op (tuning aid / evidence):
dot, GEMV, GESUMMV and the fused ATAX from 8 MiB to 8 GiB of operands, each
timed as a CUDA graph of back-to-back calls on operands rotated past L2 (best
of 3 replays); algorithmic bytes as in bench.py.  Shows where each op reaches
the HBM streaming ceiling (a launch pays a fixed ramp and tail of a few us).
usage: python tools/size_sweep.py [--quick]"""
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, os.environ.get("LIFT_ROOT") or os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import synth  # noqa: E402
import paper_conf_cgo_steuwerrd17_b200 as lift  # noqa: E402
from sweep import graph_time  # noqa: E402

dev = torch.device("cuda:0")
L2 = torch.cuda.get_device_properties(dev).L2_cache_size
pool = synth.torch_uniform(7, 0, (20 << 30) // 4, device=dev)  # 20 GiB of operand storage
SPEC = 8183.8  # GB/s, 3996 MHz x 2 x 8192 bit


def views(nbytes_each, count):
    """`count` disjoint fp32 slices of nbytes_each from the pool (cycled if the pool is short)."""
    per = nbytes_each // 4
    k = max(1, min(count, pool.numel() // per))
    return [pool[i * per:(i + 1) * per] for i in range(k)]


def run(name, bytes_per_call, make_calls, reps):
    calls = make_calls()
    t = graph_time([calls[i % len(calls)] for i in range(reps)])
    gbs = bytes_per_call / t / 1e3
    print(f"{name:28s} {bytes_per_call / 2**20:9.1f} MiB  {t:10.2f} us  {gbs:8.1f} GB/s  {100 * gbs / SPEC:5.1f} % of 8.18 TB/s",
          flush=True)


quick = "--quick" in sys.argv
r = torch.empty((), device=dev)
for lg in ([20, 22, 24, 26, 28, 30] if quick else [20, 21, 22, 23, 24, 25, 26, 27, 28, 29, 30, 31]):
    n = 1 << lg
    by = 8 * n
    sets = max(2, -(-3 * L2 // by)) if by < 3 * L2 else 1
    vs = views(4 * n, 2 * sets)
    pairs = [(vs[2 * i % len(vs)], vs[(2 * i + 1) % len(vs)]) for i in range(sets)]
    run(f"dot 2^{lg}", by, lambda: [(lambda a=a, b=b: lift.lift_dot(a, b, out=r)) for a, b in pairs],
        max(4, min(24, int(2e9 // by))))
for m, n in [(1024, 2048), (2048, 2048), (4096, 4096), (8192, 8192), (16384, 8192), (16384, 16384), (32768, 16384),
             (65536, 16384), (65536, 32768)][: (6 if quick else 9)]:
    by = 4 * m * n + 4 * (m + n)
    sets = max(2, -(-3 * L2 // by)) if by < 3 * L2 else 1
    As = [v.view(m, n) for v in views(4 * m * n, sets)]
    x = synth.torch_uniform(0, 0, n, device=dev)
    y = torch.empty(m, device=dev)
    yt = torch.empty(n, device=dev)
    reps = max(3, min(24, int(2e9 // by)))
    run(f"gemv {m}x{n}", by, lambda: [(lambda A=A: lift.lift_gemv(A, x, out=y)) for A in As], reps)
    if 2 * 4 * m * n <= pool.numel() * 4:
        Bs = [v.view(m, n) for v in views(4 * m * n, 2 * sets)]
        prs = [(Bs[2 * i % len(Bs)], Bs[(2 * i + 1) % len(Bs)]) for i in range(sets)]
        run(f"gesummv {m}x{n}", 2 * by - 4 * (m + n),
            lambda: [(lambda a=a, b=b: lift.lift_gesummv(1.5, a, 1.2, b, x, out=y)) for a, b in prs], reps)
    if n <= 16384:
        run(f"atax (fused) {m}x{n}", by + 4 * n - 4 * m,
            lambda: [(lambda A=A: lift.lift_atax(A, x, out=yt, algo="fused")) for A in As], reps)
