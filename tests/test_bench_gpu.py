"""bench.py end to end on the GPU: the contract line at N = 1, and the N > 1
code path (sharding, collectives — NCCL-style through gloo, and the fused
NVLink collectives through CUDA IPC) with two ranks sharing cuda:0 on a
shrunken workload (numbers meaningless, code path exercised)."""
import json
import os
import socket
import subprocess
import sys

import pytest

pytestmark = pytest.mark.gpu
ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def _port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def _last_json(out):
    lines = [l for l in out.splitlines() if l.startswith("{")]
    assert lines, out[-3000:]
    return json.loads(lines[-1])


def test_bench_contract_one_gpu(cuda_device):
    r = subprocess.run([sys.executable, "bench.py", "--steps", "3", "--warmup", "3", "--no-cpu", "--e2e-steps", "1",
                        "--scale", "0.05"], cwd=ROOT, capture_output=True, text=True, timeout=600)
    assert r.returncode == 0, r.stderr[-3000:]
    d = _last_json(r.stdout)
    for k in ("metric", "value", "unit", "n_gpus", "steps", "warmup", "ms_per_step", "higher_is_better", "scaling",
              "vs_baseline", "dtype", "data", "config", "roofline", "e2e", "gpu_launches", "clocks"):
        assert k in d, k
    assert d["n_gpus"] == 1 and d["steps"] == 3 and d["value"] > 0
    assert d["roofline"]["bound"] == "hbm" and d["roofline"]["achieved"] > 0
    assert d["e2e"]["h2d_bytes_per_step"] > 0 and d["gpu_launches"] == 3 * 5


@pytest.mark.parametrize("collectives", ["nccl", "fused", "auto"])
def test_bench_two_ranks_one_device(cuda_device, collectives):
    cmd = [sys.executable, "-m", "torch.distributed.run", "--nnodes=1", "--nproc-per-node", "2", "--master-addr",
           "127.0.0.1", "--master-port", str(_port()), "bench.py", "--gpus", "2", "--steps", "2", "--warmup", "3",
           "--no-cpu", "--e2e-steps", "1", "--scale", "0.02", "--test-backend", "gloo", "--test-one-device",
           "--collectives", collectives]
    r = subprocess.run(cmd, cwd=ROOT, capture_output=True, text=True, timeout=900)
    assert r.returncode == 0, (r.stdout[-2000:], r.stderr[-4000:])
    d = _last_json(r.stdout)
    want = "fused (self-checked against nccl)" if collectives == "auto" else collectives
    assert d["n_gpus"] == 2 and d["config"]["collectives"] == want and d["value"] > 0
    # fused collectives keep their epoch on the device: the timed steps are one CUDA graph as at N = 1
    assert d["config"]["launch"].startswith("cuda-graph" if collectives != "nccl" else "eager"), d["config"]["launch"]
    for name, o in d["ops"].items():  # compute-only vs the collective, per op
        assert o["compute_ms"] > 0 and o["collective_ms"] >= 0 and o["compute_GB_s_per_rank"] > 0, name
