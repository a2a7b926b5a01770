"""Time the ops whose launches overlap their predecessor's tail (tuning aid for
the L2 prefetch issued before griddepcontrol.wait): configs[0] dot 2^20,
configs[1] GEMV 4096^2, GESUMMV 4096^2 / 8192^2, ATAX 4096^2 / 8192^2, each as a
CUDA graph of back-to-back calls on operands rotated past L2 (best of 3
replays), plus the bench step's sequence [GEMV 4096^2, GESUMMV 8192^2, ATAX
8192^2] repeated; prints a checksum of each result's bits.
usage: python tools/pdl_prefetch_time.py"""
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


def bits(t):
    return zlib.crc32(t.cpu().numpy().view("uint32").tobytes())


def rotate(make, nbytes):
    sets = max(2, -(-3 * L2 // nbytes))
    return [make(k) for k in range(sets)]


# dot 2^20
n = 1 << 20
vs = rotate(lambda k: (synth.torch_uniform(2 * k, 0, n, device=dev), synth.torch_uniform(2 * k + 1, 0, n, device=dev)),
            8 * n)
out = torch.empty(1, device=dev)
b = bits(lift.lift_dot(*vs[0], out=out))
t = graph_time([(lambda v=v: lift.lift_dot(v[0], v[1], out=out)) for v in (vs * 64)[:64]])
print(f"dot 2^20:            {t:8.2f} us  {8 * n / t / 1e3:8.1f} GB/s  bits {b:08x}", flush=True)
del vs

for op, m, nn in (("gemv", 4096, 4096), ("gesummv", 4096, 4096), ("gesummv", 8192, 8192), ("atax", 4096, 4096),
                  ("atax", 8192, 8192)):
    nmat = 2 if op == "gesummv" else 1
    mats = rotate(lambda k: [synth.torch_matrix_rows(2 + 10 * k + j, nn, 0, m, device=dev) for j in range(nmat)],
                  4 * m * nn * nmat)
    x = synth.torch_uniform(0, 0, nn, device=dev)
    y = torch.empty(m if op != "atax" else nn, device=dev)

    def call(ms):
        if op == "gemv":
            return lift.lift_gemv(ms[0], x, out=y)
        if op == "gesummv":
            return lift.lift_gesummv(1.5, ms[0], 1.2, ms[1], x, out=y)
        return lift.lift_atax(ms[0], x, out=y, algo="fused")

    b = bits(call(mats[0]))
    reps = 24
    t = graph_time([(lambda ms=ms: call(ms)) for ms in (mats * reps)[:reps]])
    print(f"{op} {m}x{nn}:".ljust(21) + f"{t:8.2f} us  {4 * m * nn * nmat / t / 1e3:8.1f} GB/s  bits {b:08x}", flush=True)
    del mats

# the step's small-op sequence
G = [(synth.torch_matrix_rows(2 + k, 8192, 0, 8192, device=dev), synth.torch_matrix_rows(3 + k, 8192, 0, 8192, device=dev))
     for k in range(2)]
T = [synth.torch_matrix_rows(5 + k, 8192, 0, 8192, device=dev) for k in range(2)]
S = [synth.torch_matrix_rows(7 + k, 4096, 0, 4096, device=dev) for k in range(2)]
x8, x4 = synth.torch_uniform(0, 0, 8192, device=dev), synth.torch_uniform(1, 0, 4096, device=dev)
y8, z8, y4 = torch.empty(8192, device=dev), torch.empty(8192, device=dev), torch.empty(4096, device=dev)
calls = []
for k in range(8):
    calls += [lambda A=S[k % 2]: lift.lift_gemv(A, x4, out=y4),
              lambda A=G[k % 2][0], B=G[k % 2][1]: lift.lift_gesummv(1.5, A, 1.2, B, x8, out=y8),
              lambda A=T[k % 2]: lift.lift_atax(A, x8, out=z8)]
t = graph_time(calls) * 3
print(f"seq gemv4k+gesummv8k+atax8k: {t:8.2f} us per triple", flush=True)
