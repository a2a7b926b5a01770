"""Fused ATAX: how many ring stages to issue before the first wait (tuning aid).
Filling the whole ring at once puts ~16 MB of bulk copies in the DRAM queues
at t = 0, so every block's FIRST stage completes late; issuing P stages first
and the rest after stage 0 arrives may start the pipeline sooner.  Variant
builds (tools/variants.py) of kFusedPrologue; interleaved A/B, CUDA graphs.
usage: python tools/atax_prologue_probe.py P ...
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
for m, n in ((4096, 4096), (8192, 8192), (16384, 8192), (4096, 16384), (8192, 2048)):
    sets = max(2, int(-(-2 * l2 // (4 * m * n))) + 1)
    As = [synth.torch_matrix_rows(2 + 10 * k, n, 0, m, device=dev) for k in range(sets)]
    x = synth.torch_uniform(0, 0, n, device=dev)
    y = torch.empty(n, device=dev)
    ref = lift.lift_atax(As[0], x, algo="fused").clone()
    t = graph_time([(lambda A=A: lift.lift_atax(A, x, out=y, algo="fused")) for A in (As * 24)[:24]])
    assert torch.equal(lift.lift_atax(As[0], x, algo="fused"), ref)
    print(f"{tag:10s} atax {m}x{n}: {t:8.2f} us  {(4 * m * n + 8 * n) / t / 1e3:8.1f} GB/s", flush=True)
    del As
'''

OLD = "constexpr int kFusedPrologue = 0;"
dirs = [(f"P{p}", variant(f"atax_pro{p}", [("atax.cu", OLD, f"constexpr int kFusedPrologue = {p};")]))
        for p in sys.argv[1:]]
for rep in range(2):
    run(ROOT, TIMER, TAG="library")
    for tag, d in dirs:
        run(d, TIMER, TAG=tag)
