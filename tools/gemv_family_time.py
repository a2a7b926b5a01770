"""Time the GEMV-family configs (tuning aid): GEMV 4096^2 / 8192^2, GESUMMV 4096^2 /
8192^2 and the 8 GiB GEMV 65536 x 32768 (graph of back-to-back calls, operands
rotated past L2, best of 3 replays) and print a checksum of each result's bits.
usage: python tools/gemv_family_time.py"""
import os
import sys
import zlib

import torch

sys.path.insert(0, os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, os.environ.get("LIFT_ROOT") or os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import synth  # noqa: E402
import paper_conf_cgo_steuwerrd17_b200 as lift  # noqa: E402
from sweep import graph_time  # noqa: E402

dev = torch.device("cuda:0")
L2 = torch.cuda.get_device_properties(dev).L2_cache_size
for op, m, n, reps in (("gemv", 4096, 4096, 24), ("gemv", 8192, 8192, 24), ("gesummv", 4096, 4096, 24),
                       ("gesummv", 8192, 8192, 16), ("gemv", 65536, 32768, 3)):
    nb = (2 if op == "gesummv" else 1) * 4 * m * n
    sets = max(1, min(6, -(-3 * L2 // nb))) if nb < 4 * L2 else 1
    mats = [(synth.torch_matrix_rows(2 + 10 * k, n, 0, m, device=dev),
             synth.torch_matrix_rows(3 + 10 * k, n, 0, m, device=dev) if op == "gesummv" else None)
            for k in range(sets)]
    x = synth.torch_uniform(0, 0, n, device=dev)
    y = torch.empty(m, device=dev)

    def call(A, B):
        return lift.lift_gemv(A, x, out=y) if op == "gemv" else lift.lift_gesummv(1.5, A, 1.2, B, x, out=y)

    bits = zlib.crc32(call(*mats[0]).cpu().numpy().view("uint32").tobytes())
    t = graph_time([(lambda A=A, B=B: call(A, B)) for A, B in (mats * reps)[:reps]])
    print(f"{op} {m}x{n}: {t:9.2f} us  {nb / t / 1e3:8.1f} GB/s  bits {bits:08x}", flush=True)
    del mats
