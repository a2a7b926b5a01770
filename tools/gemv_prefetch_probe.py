"""Does an up-front L2 prefetch of the whole matrix shorten small GEMVs?
(tuning aid).  Variant builds (tools/variants.py) of k_gemv in which thread 0
of every block issues cp.async.bulk.prefetch.L2 for each of its rows at kernel
start when the matrix (A, and B for GESUMMV) is at most LIMIT MiB, so the DRAM
queues fill from the first microsecond whatever the registers in flight.
CUDA graphs of back-to-back calls on distinct copies (> 2x L2).
usage: python tools/gemv_prefetch_probe.py LIMIT_MIB ...
"""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.abspath(__file__)))
from variants import ROOT, run, variant  # noqa: E402

ANCHOR = "    const int64_t row_step = (int64_t)gridDim.x * RG;\n    int64_t row = (int64_t)blockIdx.x * RG + g;\n"
PATCH = ANCHOR + """    if (VEC == 4 && threadIdx.x == 0 && m * lda * 4 * NMAT <= (int64_t(LIMIT) << 20)) {
        for (int64_t r = (int64_t)blockIdx.x * RG; r < m; r += row_step)
            for (int gg = 0; gg < RG && r + gg < m; ++gg) {
                bulk_prefetch_l2(A + (r + gg) * lda, (uint32_t)(n * 4));
                if (NMAT == 2) bulk_prefetch_l2(B + (r + gg) * lda, (uint32_t)(n * 4));
            }
    }
"""

TIMER = r'''
import os, sys
sys.path.insert(0, os.getcwd()); sys.path.insert(0, os.path.join(os.getcwd(), "tools"))
import torch, synth
import paper_conf_cgo_steuwerrd17_b200 as lift
from sweep import graph_time
dev = torch.device("cuda:0")
l2 = torch.cuda.get_device_properties(dev).L2_cache_size
tag = os.environ["TAG"]
pool = synth.torch_uniform(2, 0, 3 << 28, device=dev)
for op, m, n in (("gemv", 4096, 4096), ("gemv", 8192, 4096), ("gemv", 8192, 8192), ("gesummv", 4096, 4096),
                 ("gesummv", 8192, 8192)):
    per = m * n * (2 if op == "gesummv" else 1)
    copies = int(-(-2 * l2 // (4 * per))) + 1
    x = pool[-n:]
    y = torch.empty(m, device=dev)
    def mk(k):
        A = pool[k * per:k * per + m * n].view(m, n)
        if op == "gemv":
            return lambda: lift.lift_gemv(A, x, out=y)
        B = pool[k * per + m * n:(k + 1) * per].view(m, n)
        return lambda: lift.lift_gesummv(1.5, A, 1.2, B, x, out=y)
    calls = [mk(k) for k in range(copies)]
    reps = max(24, copies)
    t = graph_time([calls[j % copies] for j in range(reps)])
    by = 4 * per + 4 * (m + n)
    print(f"{tag:12s} {op:8s} {m}x{n}: {t:8.2f} us  {by / t / 1e3:8.1f} GB/s", flush=True)
'''

dirs = [(f"pf<={a}MiB", variant(f"gemvpf_{a}", [("gemv.cu", ANCHOR, PATCH.replace("LIMIT", a))])) for a in sys.argv[1:]]
for rep in range(2):
    run(ROOT, TIMER, TAG="library")
    for tag, d in dirs:
        run(d, TIMER, TAG=tag)
