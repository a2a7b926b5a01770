"""k_dot launch-shape probe (tuning aid): U (float4 pairs per thread batch),
kWaves (resident waves of blocks), kUnitsPerThreadSmall (grid shrink at small
n), via patched copies (tools/variants.py).  Every variant's 2^31 result must
stay within the north_star tolerance of the library's (order changes with the
shape).  usage: python tools/dot_shape_probe.py U,WAVES,UPT ...
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
x = synth.torch_uniform(0, 0, 1 << 31, device=dev)
y = synth.torch_uniform(1, 0, 1 << 31, device=dev)
r = torch.empty((), device=dev)
for e in [int(a) for a in os.environ.get("SIZES", "20,21,22,24,26,30").split(",")]:
    n = 1 << e
    copies = int(-(-2 * l2 // (8 * n))) + 1
    if copies * n > x.numel():
        copies = 1
    sl = [(x[k * n:(k + 1) * n], y[k * n:(k + 1) * n]) for k in range(copies)]
    reps = max(24, copies) if e < 29 else 6
    t = graph_time([(lambda a=a, b=b: lift.lift_dot(a, b, out=r)) for a, b in (sl * reps)[:reps]])
    print(f"{tag:18s} dot 2^{e}: {t:9.2f} us  {8 * n / t / 1e3:8.1f} GB/s", flush=True)
'''

base = ("constexpr int kDotU = 4;", "constexpr int kWaves = 2;", "constexpr int64_t kUnitsPerThreadSmall = 2;")
# a 4th field overrides the one-wave threshold (log2 of float4 units)
shapes = [tuple(int(a) for a in v.split(",")) for v in sys.argv[1:]]
dirs = []
for sh in shapes:
    u, w, upt = sh[:3]
    new = (f"constexpr int kDotU = {u};", f"constexpr int kWaves = {w};", f"constexpr int64_t kUnitsPerThreadSmall = {upt};")
    patches = [("dot.cu", a, b) for a, b in zip(base, new)]
    tag = f"U{u} W{w} UPT{upt}"
    if len(sh) > 3:
        patches.append(("dot.cu", "constexpr int64_t kOneWaveUnits = int64_t(1) << 25;",
                        f"constexpr int64_t kOneWaveUnits = int64_t(1) << {sh[3]};"))
        tag += f" 1w<2^{sh[3]}"
    dirs.append((tag, variant("dot_" + "_".join(map(str, sh)), patches)))
for rep in range(2):
    run(ROOT, TIMER, TAG="library")
    for tag, d in dirs:
        run(d, TIMER, TAG=tag)
