"""Timing helper for the column pass (transposed SGEMV and two-pass ATAX):
run from a package root, compute both on seeded inputs, time them (12 calls
per CUDA graph on rotated copies of A, > 3x L2; median of 5 replays) and
save outputs + times to an .npz.  usage: (cd ROOT && python tools/ab_colpass.py OUT.npz)
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
for m, n in ((4096, 4096), (8192, 8192), (16384, 8192), (8192, 2048)):
    sets = max(2, -(-3 * L2 // (4 * m * n)))
    As = [synth.torch_matrix_rows(2 + 10 * k, n, 0, m, device=dev) for k in range(sets)]
    xm = synth.torch_uniform(0, 0, m, device=dev)
    x = synth.torch_uniform(0, 0, n, device=dev)
    y = torch.empty(n, device=dev)
    out[f"sgemvt_{m}x{n}"] = lift.lift_sgemv(1.0, As[0], xm, trans=True).cpu().numpy()
    out[f"atax2_{m}x{n}"] = lift.lift_atax(As[0], x, algo="twopass").cpu().numpy()
    for name, fn in (("sgemv_t", lambda A: lift.lift_sgemv(1.0, A, xm, y=y, trans=True)),
                     ("atax2p", lambda A: lift.lift_atax(A, x, out=y, algo="twopass"))):
        t = graph_time([(lambda A=A: fn(A)) for A in (As * 12)[:12]])
        out[f"t_{name}_{m}x{n}"] = np.array(t)
        print(f"{name} {m}x{n}: {t:8.2f} us", flush=True)
    del As
np.savez(sys.argv[1], **out)
