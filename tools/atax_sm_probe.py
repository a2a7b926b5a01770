"""Is the fused ATAX's main-loop skew a property of the SM (tuning aid)?

Builds the -DLIFT_TRACE library (tools/atax_trace.py), runs lift_atax (fused)
many times at each shape and records, per block, the SM it ran on (%smid) and
its "first stage arrived" / "loop done" stamps.  Prints the lateness of each SM
(loop done minus the call's median, averaged over calls), how consistent it is
between the two halves of the calls (correlation), and how much of the spread a
per-SM constant would explain.  Also a cluster probe: a kernel of 16-block
clusters (non-portable size) records which SMs share a cluster, i.e. a GPC.

usage: python tools/atax_sm_probe.py [MxN ...]"""
import ctypes
import os
import subprocess
import sys
import tempfile

import numpy as np
import torch

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
sys.path.insert(0, os.path.join(ROOT, "tools"))
import synth  # noqa: E402
from atax_trace import build_trace_lib  # noqa: E402

GPC_SRC = r'''
#include <cstdio>
#include <cuda_runtime.h>
__global__ void probe(unsigned *out) {
    unsigned smid, cid, crank;
    asm volatile("mov.u32 %0, %%smid;" : "=r"(smid));
    asm volatile("mov.u32 %0, %%clusterid.x;" : "=r"(cid));
    asm volatile("mov.u32 %0, %%cluster_ctarank;" : "=r"(crank));
    if (threadIdx.x == 0) { out[2 * blockIdx.x] = smid; out[2 * blockIdx.x + 1] = cid; }
    // hold the SM so a cluster's blocks are co-resident and distinct
    long long t0 = clock64(); while (clock64() - t0 < 2000000) {}
}
int main(int argc, char **argv) {
    int C = atoi(argv[1]);
    cudaFuncSetAttribute(probe, cudaFuncAttributeNonPortableClusterSizeAllowed, 1);
    cudaFuncSetAttribute(probe, cudaFuncAttributeMaxDynamicSharedMemorySize, 200 * 1024);
    cudaLaunchConfig_t cfg = {};
    cudaLaunchAttribute at[1];
    at[0].id = cudaLaunchAttributeClusterDimension;
    at[0].val.clusterDim.x = C; at[0].val.clusterDim.y = 1; at[0].val.clusterDim.z = 1;
    cfg.blockDim = dim3(32); cfg.dynamicSmemBytes = 200 * 1024; cfg.attrs = at; cfg.numAttrs = 1;
    int nc = 0;
    cfg.gridDim = dim3(C);
    cudaOccupancyMaxActiveClusters(&nc, (void *)probe, &cfg);
    cfg.gridDim = dim3(C * nc);
    unsigned *d; cudaMalloc(&d, 8 * C * nc);
    cudaError_t e = cudaLaunchKernelEx(&cfg, probe, d);
    cudaDeviceSynchronize();
    unsigned h[4096]; cudaMemcpy(h, d, 8 * C * nc, cudaMemcpyDeviceToHost);
    printf("%d %d %s\n", C, nc, cudaGetErrorString(e));
    for (int i = 0; i < C * nc; ++i) printf("%u %u\n", h[2 * i], h[2 * i + 1]);
    return 0;
}
'''


def gpc_map(d):
    src = os.path.join(d, "gpc.cu")
    open(src, "w").write(GPC_SRC)
    exe = os.path.join(d, "gpc")
    subprocess.check_call(["nvcc", "-gencode", "arch=compute_100a,code=sm_100a", "-o", exe, src])
    for C in (16, 8):
        out = subprocess.run([exe, str(C)], capture_output=True, text=True).stdout.split("\n")
        head = out[0].split()
        print(f"cluster probe C={C}: {head[1]} clusters co-resident ({' '.join(head[2:])})")
        groups = {}
        for line in out[1:]:
            if line.strip():
                sm, cid = (int(v) for v in line.split())
                groups.setdefault(cid, []).append(sm)
        for cid in sorted(groups):
            print(f"  cluster {cid:3d}: SMs {sorted(groups[cid])}")


def main():
    shapes = [tuple(int(v) for v in a.split("x")) for a in sys.argv[1:]] or [(8192, 8192)]
    dev = torch.device("cuda:0")
    with tempfile.TemporaryDirectory() as d:
        gpc_map(d)
        L = ctypes.CDLL(build_trace_lib(d))
        L.lift_atax_workspace_bytes.restype = ctypes.c_size_t
        L.lift_atax_workspace_bytes.argtypes = [ctypes.c_int64, ctypes.c_int64]
        L.lift_atax_algo_run.argtypes = [ctypes.c_int, ctypes.c_int64, ctypes.c_int64] + [ctypes.c_void_p] * 4 + \
            [ctypes.c_size_t, ctypes.c_void_p]
        L.lift_trace_copy.argtypes = [ctypes.c_void_p, ctypes.c_size_t]
        for m, n in shapes:
            As = [synth.torch_matrix_rows(2 + k, n, 0, m, device=dev) for k in range(3)]
            x = synth.torch_uniform(0, 0, n, device=dev)
            y = torch.empty(n, device=dev)
            ws = torch.zeros(L.lift_atax_workspace_bytes(m, n), dtype=torch.uint8, device=dev)
            s = torch.cuda.current_stream().cuda_stream
            G = min(torch.cuda.get_device_properties(dev).multi_processor_count, m)
            calls = 40
            late = np.zeros((calls, 256)) * np.nan
            first = np.zeros((calls, 256)) * np.nan
            sm_of_block = []
            for it in range(calls + 4):
                assert L.lift_atax_algo_run(1, m, n, As[it % 3].data_ptr(), x.data_ptr(), y.data_ptr(),
                                            ws.data_ptr(), ws.numel(), s) == 0
                torch.cuda.synchronize()
                buf = np.zeros(256 * 16, dtype=np.uint64)
                assert L.lift_trace_copy(buf.ctypes.data, buf.nbytes) == 0
                t = buf.reshape(256, 16)[:G].astype(np.int64)
                if it < 4:
                    continue
                sm = t[:, 15]
                sm_of_block.append(sm.copy())
                loop = (t[:, 3] - t[:, 0].min()) / 1e3
                fs = (t[:, 1] - t[:, 0].min()) / 1e3
                late[it - 4, sm] = loop - np.median(loop)
                first[it - 4, sm] = fs - np.median(fs)
            S = np.stack(sm_of_block)
            same_map = bool((S == S[0]).all())
            print(f"== atax {m}x{n}: {G} blocks, {calls} calls; block->SM map identical in every call: {same_map}")
            used = ~np.isnan(late).all(0)
            a, b = np.nanmean(late[0::2], 0)[used], np.nanmean(late[1::2], 0)[used]
            print(f"  per-SM lateness (loop done - call median), us: spread of the mean {a.min():.2f} .. {a.max():.2f};"
                  f" correlation between even and odd calls {np.corrcoef(a, b)[0, 1]:.3f}")
            fa, fb = np.nanmean(first[0::2], 0)[used], np.nanmean(first[1::2], 0)[used]
            print(f"  per-SM first-stage lateness: spread {fa.min():.2f} .. {fa.max():.2f}; even/odd correlation "
                  f"{np.corrcoef(fa, fb)[0, 1]:.3f}")
            resid = late[:, used] - np.nanmean(late[:, used], 0)
            print(f"  per-call spread (max - min over SMs) median {np.median(np.nanmax(late, 1) - np.nanmin(late, 1)):.2f} us;"
                  f" after removing each SM's mean lateness {np.median(resid.max(1) - resid.min(1)):.2f} us")
            order = np.argsort(np.nanmean(late, 0))
            ids = [i for i in order if used[i]]
            mean = np.nanmean(late, 0)
            print("  latest SMs (smid: mean lateness us):", ", ".join(f"{i}:{mean[i]:+.2f}" for i in ids[-20:]))
            print("  earliest SMs:", ", ".join(f"{i}:{mean[i]:+.2f}" for i in ids[:20]))
            print("  all SMs by smid:", " ".join(f"{mean[i]:+.1f}" if used[i] else "nan" for i in range(int(S.max()) + 1)))


if __name__ == "__main__":
    main()
