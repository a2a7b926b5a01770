"""A/B helper for the fused ATAX kernel: run from a package root (this tree or
an exported older commit), compute lift_atax(algo="fused") on seeded inputs at
the Table-1 / configs shapes, time it (12 calls per CUDA graph, every call on
its own copy of A, copies > 2x L2; median of 5 replays) and save outputs and
times to an .npz so two builds can be compared bit for bit.
usage: (cd ROOT && python /path/to/tools/ab_atax.py OUT.npz)
"""
import os
import sys

import numpy as np
import torch

sys.path.insert(0, os.getcwd())
sys.path.insert(0, os.path.join(os.getcwd(), "tools"))
import synth  # noqa: E402
import paper_conf_cgo_steuwerrd17_b200 as lift  # noqa: E402
from sweep import graph_time  # noqa: E402

dev = torch.device("cuda:0")
L2 = torch.cuda.get_device_properties(dev).L2_cache_size
out = {}
for m, n in ((2048, 2048), (4096, 4096), (8192, 8192), (16384, 8192), (8192, 16384), (4096, 1024), (1000, 300 * 4)):
    sets = max(2, -(-3 * L2 // (4 * m * n)))
    As = [synth.torch_matrix_rows(2 + 10 * k, n, 0, m, device=dev) for k in range(sets)]
    x = synth.torch_uniform(0, 0, n, device=dev)
    y = torch.empty(n, device=dev)
    out[f"y_{m}x{n}"] = lift.lift_atax(As[0], x, algo="fused").cpu().numpy()
    calls = [(lambda A=A: lift.lift_atax(A, x, out=y, algo="fused")) for A in (As * 12)[:12]]
    t = graph_time(calls)
    out[f"t_{m}x{n}"] = np.array(t)
    print(f"atax {m}x{n}: {t:8.2f} us  {4 * m * n / t / 1e3:8.1f} GB/s", flush=True)
    del As
np.savez(sys.argv[1], **out)
