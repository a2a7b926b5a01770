"""Time pairs of the bench step's ops back to back in one CUDA graph (tuning aid):
e.g. ATAX 8192^2 followed by the 8 GiB GEMV, to see how one op's launch mode
affects its neighbour (programmatic dependent launch, cooperative launches).
usage: python tools/step_pairs_time.py"""
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, os.environ.get("LIFT_ROOT") or os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import synth  # noqa: E402
import paper_conf_cgo_steuwerrd17_b200 as lift  # noqa: E402
from sweep import graph_time  # noqa: E402

dev = torch.device("cuda:0")
T = synth.torch_matrix_rows(5, 8192, 0, 8192, device=dev)
G = synth.torch_matrix_rows(6, 8192, 0, 8192, device=dev), synth.torch_matrix_rows(7, 8192, 0, 8192, device=dev)
Big = synth.torch_matrix_rows(8, 32768, 0, 16384, device=dev)  # 2 GiB GEMV
x8, x32 = synth.torch_uniform(0, 0, 8192, device=dev), synth.torch_uniform(1, 0, 32768, device=dev)
d = synth.torch_uniform(2, 0, 1 << 28, device=dev)
y8, z8, y16 = torch.empty(8192, device=dev), torch.empty(8192, device=dev), torch.empty(16384, device=dev)
s = torch.empty((), device=dev)
ops = {
    "atax": lambda: lift.lift_atax(T, x8, out=z8),
    "gesummv": lambda: lift.lift_gesummv(1.5, G[0], 1.2, G[1], x8, out=y8),
    "gemv2G": lambda: lift.lift_gemv(Big, x32, out=y16),
    "dot1G": lambda: lift.lift_dot(d, d, out=s),
}
seqs = [["atax"], ["gemv2G"], ["dot1G"], ["gesummv"], ["atax", "gemv2G"], ["gesummv", "atax"], ["atax", "dot1G"],
        ["gesummv", "atax", "gemv2G", "dot1G"]]
for seq in seqs:
    t = graph_time([ops[k] for _ in range(4) for k in seq]) * len(seq)
    print(f"{' -> '.join(seq):34s} {t:9.2f} us per sequence", flush=True)
