"""Hand-off fences: k_dot's last-block ticket (atom.acq_rel vs __threadfence +
atomicAdd) and the fused ATAX grid barrier's arrival (red.release vs
__threadfence + atomicAdd), tuning aid.  Interleaved A/B over patched copies
(tools/variants.py); CUDA graphs of back-to-back calls on distinct operands.
usage: python tools/fence_probe.py
"""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.abspath(__file__)))
from variants import ROOT, run, variant  # noqa: E402

TIMER = r'''
import os, sys
sys.path.insert(0, os.getcwd()); sys.path.insert(0, os.path.join(os.getcwd(), "tools"))
import torch, synth
import paper_conf_cgo_steuwerrd17_b200 as lift
from sweep import graph_time
dev = torch.device("cuda:0")
l2 = torch.cuda.get_device_properties(dev).L2_cache_size
tag = os.environ["TAG"]
x = synth.torch_uniform(0, 0, 1 << 28, device=dev)
y = synth.torch_uniform(1, 0, 1 << 28, device=dev)
r = torch.empty((), device=dev)
for e in (20, 22, 24, 27):
    n = 1 << e
    copies = int(-(-2 * l2 // (8 * n))) + 1
    sl = [(x[k * n:(k + 1) * n], y[k * n:(k + 1) * n]) for k in range(copies)]
    reps = max(24, copies)
    t = graph_time([(lambda a=a, b=b: lift.lift_dot(a, b, out=r)) for a, b in (sl * reps)[:reps]])
    print(f"{tag:10s} dot  2^{e}: {t:8.2f} us", flush=True)
for m, n in ((148, 8192), (4096, 4096), (8192, 8192)):
    sets = max(2, int(-(-2 * l2 // (4 * m * n))) + 1)
    As = [synth.torch_matrix_rows(2 + 10 * k, n, 0, m, device=dev) for k in range(sets)]
    xa = synth.torch_uniform(0, 0, n, device=dev)
    ya = torch.empty(n, device=dev)
    t = graph_time([(lambda A=A: lift.lift_atax(A, xa, out=ya, algo="fused")) for A in (As * 24)[:24]])
    print(f"{tag:10s} atax {m}x{n}: {t:8.2f} us", flush=True)
    del As
'''

OLD = [("dot.cu", "constexpr bool kDotAcqRelTicket = true;", "constexpr bool kDotAcqRelTicket = false;"),
       ("atax.cu", "constexpr bool kGridReleaseArrive = true;", "constexpr bool kGridReleaseArrive = false;")]
d_old = variant("fences_old", OLD)
for rep in range(2):
    run(ROOT, TIMER, TAG="new")
    run(d_old, TIMER, TAG="old")
