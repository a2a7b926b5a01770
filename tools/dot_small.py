"""k_dot at small n over distinct slices (graph of >= 20 calls).  usage: python tools/dot_small.py"""
import os, sys
import torch
sys.path.insert(0, "/root/repo"); sys.path.insert(0, "/root/repo/tools")
import synth
import paper_conf_cgo_steuwerrd17_b200 as lift
from sweep import graph_time
dev = torch.device("cuda:0")
dx = synth.torch_uniform(0, 0, 40 << 20, device=dev)
dy = synth.torch_uniform(1, 0, 40 << 20, device=dev)
for n in (1 << 16, 1 << 18, 1 << 20, 1 << 22, 1 << 24):
    copies = max(2, min(40, (300 << 20) // (8 * n)))
    res = torch.empty((), device=dev)
    calls = [(lambda k=k, n=n: lift.lift_dot(dx[k * n:(k + 1) * n], dy[k * n:(k + 1) * n], out=res)) for k in range(copies)]
    reps = max(20, copies)
    t = graph_time([calls[j % copies] for j in range(reps)])
    print(f"n=2^{n.bit_length()-1:2d}: {t:7.2f} us  {8*n/t/1e3:7.1f} GB/s", flush=True)
