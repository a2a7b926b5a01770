"""Small dots in a CUDA graph (tuning aid): dot 2^16 .. 2^25, back-to-back calls on
distinct slices rotated past L2, best of 3 replays.  usage: python tools/dot_small_time.py"""
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, os.environ.get("LIFT_ROOT") or os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import synth  # noqa: E402
import paper_conf_cgo_steuwerrd17_b200 as lift  # noqa: E402
from sweep import graph_time  # noqa: E402

dev = torch.device("cuda:0")
pool = synth.torch_uniform(7, 0, (1 << 30) // 4, device=dev)  # 1 GiB
r = torch.empty((), device=dev)
for lg in (16, 18, 20, 21, 22, 23, 24, 25):
    n = 1 << lg
    k = min(48, pool.numel() // (2 * n))
    sl = [(pool[2 * i * n:(2 * i + 1) * n], pool[(2 * i + 1) * n:(2 * i + 2) * n]) for i in range(k)]
    t = graph_time([(lambda a=a, b=b: lift.lift_dot(a, b, out=r)) for a, b in (sl * 48)[:48]])
    print(f"dot 2^{lg}: {t:8.2f} us  {8 * n / t / 1e3:8.1f} GB/s", flush=True)
