"""bench.py pieces that need no GPU: the workload matches BASELINE.json, the
algorithmic byte counts match DESIGN.md §5, and the reference arm (the fp64
oracle on the host cores) prints a contract line."""
import json
import os
import subprocess
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import bench  # noqa: E402


def test_workload_is_baseline_configs_1_to_4():
    cfg = json.load(open(os.path.join(ROOT, "BASELINE.json")))["configs"]
    idx = {w[3] for w in bench.WORKLOAD}
    assert idx == {1, 2, 3, 4}
    shapes = {w[0]: w[2] for w in bench.WORKLOAD}
    assert "4096" in cfg[1] and shapes["gemv_4096x4096"] == dict(m=4096, n=4096)
    assert "8192" in cfg[2] and shapes["gesummv_8192x8192"] == dict(m=8192, n=8192)
    assert "8192" in cfg[3] and shapes["atax_8192x8192"] == dict(m=8192, n=8192)
    assert "65536" in cfg[4] and shapes["gemv_65536x32768"] == dict(m=65536, n=32768)
    assert "2^31" in cfg[4] and shapes["dot_2^31"] == dict(n=1 << 31)


def test_algorithmic_bytes():
    assert bench.alg_bytes("dot", dict(n=1 << 31)) == 17179869188
    assert bench.alg_bytes("gemv", dict(m=4096, n=4096)) == 67141632
    assert bench.alg_bytes("gemv", dict(m=65536, n=32768)) == 8590327808
    assert bench.alg_bytes("gesummv", dict(m=8192, n=8192)) == 536936448
    assert bench.alg_bytes("atax", dict(m=8192, n=8192)) == 268500992
    assert bench.alg_bytes("atax", dict(m=8192, n=8192), "twopass") == 537001984
    # NEXT-3: x, y read, z[n/128] written; iterated: 2^28 -> 2^21 -> 16384 -> 128 -> 1 partials
    assert bench.alg_bytes("partial_dot", dict(n=1 << 20)) == 8 * (1 << 20) + 4 * 8192
    stages = [1 << 21, 1 << 14, 1 << 7, 1]
    assert bench.alg_bytes("dot_listing1", dict(n=1 << 28)) == (
        8 * (1 << 28) + 4 * stages[0] + sum(4 * a + 4 * b for a, b in zip(stages, stages[1:])))
    # NEXT-4 transposed SGEMV: A, x[m] read, y[n] written (and read when beta != 0)
    assert bench.alg_bytes("sgemv_t", dict(m=8192, n=4096, beta=0.0)) == 4 * 8192 * 4096 + 4 * 8192 + 4 * 4096
    assert bench.alg_bytes("sgemv_t", dict(m=8192, n=4096, beta=0.5)) == 4 * 8192 * 4096 + 4 * 8192 + 8 * 4096


def test_reference_arm_contract_line():
    r = subprocess.run([sys.executable, "bench.py", "--impl", "reference", "--steps", "1", "--warmup", "1"], cwd=ROOT,
                       capture_output=True, text=True, timeout=600)
    assert r.returncode == 0, r.stderr[-2000:]
    d = json.loads([l for l in r.stdout.splitlines() if l.startswith("{")][-1])
    assert d["impl"] == "reference" and d["value"] > 0 and d["unit"] == "GB/s"
    assert d["e2e"]["h2d_bytes_per_step"] == 0 and d["e2e"]["value"] == d["value"]
    assert d["cpu_baseline"]["kind"] == "oracle" and d["cpu_baseline"]["cores"] >= 1
    assert d["config"]["workload"] == bench.WORKLOAD_NAME


def test_peaks():
    # measured copy peak from the driver's file; theoretical HBM3e peak from its memory clock
    peak, src = bench.measured_peak()
    assert peak > 1000 and src
    assert abs(bench.spec_peak() - 3996e6 * 2 * 8192 / 8 / 1e9) < 50


def test_table1_sizes_cover_paper_and_configs0():
    """bench.py's table1 block: configs[0]'s dot and the paper's small / large
    matrix sizes (Table 1: 4K^2 and 8K^2) for every matrix op."""
    names = {t[0] for t in bench.TABLE1}
    assert "dot_2^20" in names
    for op in ("gemv", "gesummv", "atax"):
        for s in (4096, 8192):
            assert f"{op}_{s}x{s}" in names
    cfg0 = json.load(open(os.path.join(ROOT, "BASELINE.json")))["configs"][0]
    assert "1,048,576" in cfg0 and dict(bench.TABLE1[0][2]) == dict(n=1 << 20)


def test_table1_calls_bind_their_own_operands(monkeypatch):
    """Every call of every size reads a distinct slice of its own size (no late
    binding of loop variables), and the slices of one size do not overlap."""
    import torch

    monkeypatch.setattr(bench, "TABLE1", [("dot_64", "dot", dict(n=64), "fused"),
                                          ("gemv_8x16", "gemv", dict(m=8, n=16), "fused"),
                                          ("gesummv_4x8", "gesummv", dict(m=4, n=8), "fused"),
                                          ("atax_8x4", "atax", dict(m=8, n=4), "twopass"),
                                          ("partial_dot_256", "partial_dot", dict(n=256), None),
                                          ("dot_listing1_128", "dot_listing1", dict(n=128), None),
                                          ("sgemv_t_8x4", "sgemv_t", dict(m=8, n=4, beta=0.5), None)])
    seen = []

    class Stub:
        def lift_dot(self, x, y, out):
            seen.append(("dot", x.numel(), x.data_ptr(), y.numel()))

        def lift_gemv(self, A, x, out):
            seen.append(("gemv", tuple(A.shape), A.data_ptr(), x.numel()))

        def lift_gesummv(self, a, A, b, B, x, out):
            assert B.data_ptr() == A.data_ptr() + 4 * A.numel() and a == bench.ALPHA and b == bench.BETA
            seen.append(("gesummv", tuple(A.shape), A.data_ptr(), x.numel()))

        def lift_atax(self, A, x, out, algo):
            assert algo == "twopass"
            seen.append(("atax", tuple(A.shape), A.data_ptr(), x.numel()))

        def lift_partial_dot(self, x, y, out):
            assert out.numel() == x.numel() // 128
            seen.append(("partial_dot", x.numel(), x.data_ptr(), y.numel()))

        def lift_dot_listing1(self, x, y, out):
            seen.append(("dot_listing1", x.numel(), x.data_ptr(), y.numel()))

        def lift_sgemv(self, alpha, A, x, beta, y, trans):
            assert trans and beta == 0.5 and y.numel() == A.shape[1]
            seen.append(("sgemv_t", tuple(A.shape), A.data_ptr(), x.numel()))

    pool, dx, dy = torch.zeros(1 << 16), torch.zeros(1 << 12), torch.zeros(1 << 12)
    sets = bench.table1_calls(Stub(), pool, dx, dy, torch.device("cpu"), l2_bytes=1000)
    for name, op, shp, algo, calls in sets:
        seen.clear()
        for c in calls:
            c()
        assert len(calls) >= 2 and len({s[2] for s in seen}) == len(calls), name
        for s in seen:
            if op in ("dot", "partial_dot", "dot_listing1"):
                assert s[1] == s[3] == shp["n"]
            elif op == "sgemv_t":
                assert s[1] == (shp["m"], shp["n"]) and s[3] == shp["m"]
            else:
                assert s[1] == (shp["m"], shp["n"]) and s[3] == shp["n"]


def test_clock_rejection_rule():
    """The contract's rejection rule on the NVML samples of a timed region:
    thermal / hardware slowdowns reject, sw_power_cap is kept (and noted), and
    clocks far below max with no reason (a leftover clock lock) reject."""
    def sampler(samples, reasons, max_mhz=1965):
        s = bench.ClockSampler.__new__(bench.ClockSampler)
        s.ok, s.samples, s.reasons, s.max_mhz = True, samples, reasons, max_mhz
        return s

    assert not sampler([1950, 1965], 0).rejectable()
    assert not sampler([1800, 1810], 0x4).rejectable()          # sw_power_cap: kept
    assert "sw_power_cap" in sampler([1800], 0x4).summary()["reasons"]
    assert sampler([1900], 0x8).rejectable()                    # hw_slowdown
    assert sampler([1900], 0x20).rejectable()                   # sw_thermal_slowdown
    assert sampler([1900], 0x40 | 0x4).rejectable()             # hw_thermal_slowdown
    assert sampler([1000, 1005], 0).rejectable()                # stuck low, no reason
    assert not sampler([1000, 1005], 0x4).rejectable()          # low but power-capped: noted, kept
    assert sampler([1000], 0x1).rejectable()                    # gpu_idle is not a reason: low clocks reject
    s = bench.ClockSampler.__new__(bench.ClockSampler)
    s.ok, s.samples, s.reasons, s.max_mhz = False, [], 0, None
    assert not s.rejectable()                                   # NVML unavailable: nothing to judge
