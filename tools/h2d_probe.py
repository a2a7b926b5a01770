"""Pinned host -> device copy bandwidth: one stream vs several, chunk sizes (e2e ceiling)."""
import torch

dev = torch.device("cuda:0")
N = 1 << 28  # 1 GiB of fp32
h = torch.empty(N, dtype=torch.float32, pin_memory=True)
h.uniform_()
d = torch.empty(N, dtype=torch.float32, device=dev)
for nstreams in (1, 2, 4):
    for chunk_mib in (64, 256, 1024):
        streams = [torch.cuda.Stream(device=dev) for _ in range(nstreams)]
        ch = min(N, chunk_mib << 18)
        best = 0.0
        for _ in range(4):
            torch.cuda.synchronize()
            s0 = torch.cuda.Event(enable_timing=True)
            e0 = torch.cuda.Event(enable_timing=True)
            s0.record()
            for i, o in enumerate(range(0, N, ch)):
                st = streams[i % nstreams]
                st.wait_event(s0)
                with torch.cuda.stream(st):
                    d[o:o + ch].copy_(h[o:o + ch], non_blocking=True)
            for st in streams:
                torch.cuda.current_stream().wait_stream(st)
            e0.record()
            torch.cuda.synchronize()
            best = max(best, 4 * N / (s0.elapsed_time(e0) * 1e-3) / 1e9)
        print(f"H2D streams {nstreams} chunk {chunk_mib:5d} MiB: {best:6.1f} GB/s", flush=True)
