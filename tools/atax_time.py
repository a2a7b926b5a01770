"""Time lift_atax(algo="fused") at the Table-1 / configs shapes (tuning aid):
24 calls per CUDA graph, every call on its own copy of A (copies > 2x L2), best
of 3 replays; also checks each result against the oracle once.
usage: python tools/atax_time.py [MxN ...]"""
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.abspath(__file__)))
# LIFT_ROOT: the package root to time (tools/ab_tree.sh points it at an older tree)
sys.path.insert(0, os.environ.get("LIFT_ROOT") or os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import oracle  # noqa: E402
import synth  # noqa: E402
import paper_conf_cgo_steuwerrd17_b200 as lift  # noqa: E402
from sweep import graph_time  # noqa: E402

dev = torch.device("cuda:0")
L2 = torch.cuda.get_device_properties(dev).L2_cache_size
shapes = [tuple(int(v) for v in a.split("x")) for a in sys.argv[1:]] or \
    [(4096, 4096), (8192, 8192), (2048, 2048), (16384, 8192), (148, 8192), (8192, 16384), (8192, 32768)]
for m, n in shapes:
    sets = max(2, -(-3 * L2 // (4 * m * n)))
    As = [synth.torch_matrix_rows(2 + 10 * k, n, 0, m, device=dev) for k in range(sets)]
    x = synth.torch_uniform(0, 0, n, device=dev)
    y = torch.empty(n, device=dev)
    got = lift.lift_atax(As[0], x, algo="fused").cpu().numpy()
    ok, margin = oracle.within_tol(got, *oracle.atax(As[0].cpu().numpy(), x.cpu().numpy()))
    t = graph_time([(lambda A=A: lift.lift_atax(A, x, out=y, algo="fused")) for A in (As * 24)[:24]])
    import zlib
    crc = zlib.crc32(got.view("uint32").tobytes())  # compare the exact bits across builds / settings
    print(f"atax {m}x{n}: {t:8.2f} us  {4 * m * n / t / 1e3:8.1f} GB/s  parity {'ok' if ok else 'BAD'} {margin:.2g}"
          f"  bits {crc:08x}", flush=True)
    del As
