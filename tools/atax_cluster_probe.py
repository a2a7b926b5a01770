"""Fused-ATAX second stage: grid barrier (cluster=1) against clusters of
2/4/8/16 blocks reducing through distributed shared memory (cluster=C).

Each timed call reads a different copy of A (copies totalling > 2x L2), so
every call streams A from HBM; time per call from a CUDA graph of 12 calls
(tools/sweep.graph_time: median of 5 replays).
usage: python tools/atax_cluster_probe.py
"""
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
sys.path.insert(0, os.path.dirname(os.path.abspath(__file__)))
import synth  # noqa: E402
import paper_conf_cgo_steuwerrd17_b200 as lift  # noqa: E402
from sweep import graph_time  # noqa: E402

dev = torch.device("cuda:0")
L2 = torch.cuda.get_device_properties(dev).L2_cache_size
print(f"# {torch.cuda.get_device_name(dev)}  SMs {torch.cuda.get_device_properties(dev).multi_processor_count}"
      f"  L2 {L2 >> 20} MiB", flush=True)
for m, n in ((2048, 2048), (4096, 4096), (8192, 8192), (16384, 8192), (8192, 16384), (4096, 1024)):
    sets = max(2, -(-3 * L2 // (4 * m * n)))
    As = [synth.torch_matrix_rows(2 + 10 * k, n, 0, m, device=dev) for k in range(sets)]
    x = synth.torch_uniform(0, 0, n, device=dev)
    y = torch.empty(n, device=dev)
    ref = lift.lift_atax(As[0], x, algo="fused").clone()
    for clu in (1, 2, 4, 8, 16):
        try:
            got = lift.lift_atax_fused_tuned(As[0], x, cluster=clu)
        except lift.LiftError as e:
            print(f"atax {m}x{n} cluster {clu}: {e}", flush=True)
            continue
        err = (got - ref).abs().max().item() / ref.abs().max().item()
        assert err < 1e-5, (clu, err)  # a different summation order than the automatic setting
        calls = [(lambda A=A: lift.lift_atax_fused_tuned(A, x, out=y, cluster=clu)) for A in (As * 12)[:12]]
        t = graph_time(calls)
        print(f"atax {m}x{n} cluster {clu:2d}: {t:8.2f} us  {4 * m * n / t / 1e3:8.1f} GB/s", flush=True)
    del As
