"""Timeline of the single-block fused ATAX (tuning aid): builds a variant of
liblift.so with -DLIFT_TRACE (globaltimer stamps by thread 0 of every block at
the kernel's phase boundaries; the product library has none), runs lift_atax
through its C ABI at the given shapes and prints, per phase boundary, the
spread of the blocks' stamps relative to the earliest block start:

  0 start (after griddepcontrol.wait)   1 first ring stage arrived
  2 half of the block's stages done     3 main loop done (last rank-1 update)
  4 partial row stored                  5 grid barrier passed
  6 column slice summed                 7 column sum's loads consumed (first pass)
  8 (LIFT_TRACE_REPEAT=1) the same loads repeated once more: pure L2-hit latency

usage: python tools/atax_trace.py [MxN ...]"""
import ctypes
import os
import subprocess
import sys
import tempfile

import numpy as np
import torch

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import synth  # noqa: E402
from paper_conf_cgo_steuwerrd17_b200 import build as B  # noqa: E402

NAMES = ["start", "first stage", "half stages", "loop done", "P stored", "barrier out", "colsum done",
         "colsum loads", "repeat loads"]


REPEAT = os.environ.get("LIFT_TRACE_REPEAT") == "1"  # also time a repeat of the column-sum loads
NS = 9 if REPEAT else 8


def build_trace_lib(d):
    objs = []
    extra = ["-DLIFT_TRACE_REPEAT"] if REPEAT else []
    for u in B.UNITS:
        o = os.path.join(d, u.replace(".cu", ".o"))
        subprocess.check_call([B._nvcc(), *B.NVCC_FLAGS, "-DLIFT_TRACE", *extra, "-c", os.path.join(B.CSRC, u), "-o", o])
        objs.append(o)
    so = os.path.join(d, "liblift_trace.so")
    subprocess.check_call([B._nvcc(), *B.ARCH, "-shared", "-cudart", "static", "-o", so, *objs])
    return so


def main():
    shapes = [tuple(int(v) for v in a.split("x")) for a in sys.argv[1:]] or [(8192, 8192), (4096, 4096)]
    dev = torch.device("cuda:0")
    with tempfile.TemporaryDirectory() as d:
        L = ctypes.CDLL(build_trace_lib(d))
        L.lift_atax_workspace_bytes.restype = ctypes.c_size_t
        L.lift_atax_workspace_bytes.argtypes = [ctypes.c_int64, ctypes.c_int64]
        L.lift_atax_algo_run.argtypes = [ctypes.c_int, ctypes.c_int64, ctypes.c_int64] + [ctypes.c_void_p] * 4 + \
            [ctypes.c_size_t, ctypes.c_void_p]
        L.lift_trace_copy.argtypes = [ctypes.c_void_p, ctypes.c_size_t]
        for m, n in shapes:
            sets = 3
            As = [synth.torch_matrix_rows(2 + k, n, 0, m, device=dev) for k in range(sets)]
            x = synth.torch_uniform(0, 0, n, device=dev)
            y = torch.empty(n, device=dev)
            ws = torch.zeros(L.lift_atax_workspace_bytes(m, n), dtype=torch.uint8, device=dev)
            s = torch.cuda.current_stream().cuda_stream
            G = torch.cuda.get_device_properties(dev).multi_processor_count
            G = min(G, m)
            runs = []
            for it in range(12):
                A = As[it % sets]
                assert L.lift_atax_algo_run(1, m, n, A.data_ptr(), x.data_ptr(), y.data_ptr(), ws.data_ptr(),
                                            ws.numel(), s) == 0
                torch.cuda.synchronize()
                buf = np.zeros(256 * 16, dtype=np.uint64)
                assert L.lift_trace_copy(buf.ctypes.data, buf.nbytes) == 0
                t = buf.reshape(256, 16)[:G, :NS].astype(np.int64)
                runs.append(t - t[:, 0].min())
            print(f"== atax {m}x{n}: {G} blocks, stamps in us after the earliest block start "
                  f"(median over the last 8 of 12 calls; min / median / max over blocks)")
            R = np.stack(runs[4:])  # calls, blocks, phases
            for k, name in enumerate(NAMES[:NS]):
                v = R[:, :, k] / 1e3
                print(f"  {k} {name:12s}  min {np.median(v.min(1)):7.2f}  med {np.median(np.median(v, 1)):7.2f}"
                      f"  max {np.median(v.max(1)):7.2f}")
            # rows per block (cyclic stages of CR rows): does the main-loop skew follow the row count?
            loop = np.median(R[:, :, 3], 0) / 1e3
            cnt = np.array([len(range(b, m, G)) for b in range(G)])  # rows when CR = 1 (n > 4096)
            for c in sorted(set(cnt)):
                sel = cnt == c
                print(f"  blocks with {c} rows (CR=1 count): {sel.sum():3d}, loop done median {np.median(loop[sel]):.2f}"
                      f" max {loop[sel].max():.2f}")
            late = np.argsort(loop)[-8:]
            print(f"  latest blocks (loop done): {sorted(late.tolist())}")
            g = np.unique(np.diff(np.sort(R.reshape(-1))))
            print(f"  globaltimer granularity: smallest nonzero step {g[g > 0].min() if (g > 0).any() else 0} ns")


if __name__ == "__main__":
    main()
