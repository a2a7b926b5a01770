"""Fused-ATAX launch-shape variants (tuning aid; the library is not changed).

Each variant is a copy of the package under /tmp with textual patches to
csrc/atax.cu, built and timed by tools/ab_atax.py (bitwise outputs saved, so
the variants that keep the summation order can be checked against the
library).  usage: python tools/atax_variant_probe.py [name ...]
"""
import os
import shutil
import subprocess
import sys

import numpy as np

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
SRC = os.path.join(ROOT, "paper_conf_cgo_steuwerrd17_b200", "csrc", "atax.cu")

CASES = ("    LIFT_FUSED_CASE(1, 4)\n", "    LIFT_FUSED_CASE(1, 4)\n    LIFT_FUSED_CASE(2, 4)\n")
VARIANTS = {
    "lib": [],
    # QC = 2 (n in (2048, 4096]) with 4 rows per step: one barrier per 64 KiB stage
    "qc2cr4": [("const int cr_max = qc == 1 ? 4 : (qc == 2 ? 2 : 1);", "const int cr_max = qc <= 2 ? 4 : 1;"),
               ("constexpr size_t kFusedStageTarget = 32 * 1024;", "constexpr size_t kFusedStageTarget = 64 * 1024;"),
               ("constexpr size_t kFusedRingTarget = 112 * 1024;", "constexpr size_t kFusedRingTarget = 128 * 1024;"),
               CASES],
    # deeper ring (more bytes in flight per SM)
    "ring160": [("constexpr size_t kFusedRingTarget = 112 * 1024;", "constexpr size_t kFusedRingTarget = 160 * 1024;")],
    # column pass (transposed SGEMV, two-pass ATAX): fewer row splits, more rows per block
    "splits_div2": [("    int64_t S = (int64_t)d.sms * per_sm / cblocks;", "    int64_t S = (int64_t)d.sms * per_sm / cblocks / 2;")],
    "splits_x2": [("    int64_t S = (int64_t)d.sms * per_sm / cblocks;", "    int64_t S = (int64_t)d.sms * per_sm / cblocks * 2;")],
    "splits_div4": [("    int64_t S = (int64_t)d.sms * per_sm / cblocks;", "    int64_t S = (int64_t)d.sms * per_sm / cblocks / 4;")],
    # wide-row cluster kernel with NO cross-block exchange (no arm, push or wait; WRONG results):
    # the data path alone (ring, bulk copies, dots, updates) on the cluster launch
    "wide_alone": [("            mbar_wait_parity(sfull + psb, psphase);  // every block's group k-1 sums are here", ""),
                   ("                    st_async_dsmem1(dsmem_addr_raw(la, (uint32_t)(b + li)), dr, dsmem_addr_raw(lb, (uint32_t)(b + li)));",
                    "                    if (dr == 1234.5f) sums[0] = dr;"),
                   ("        if (tid == 0 && rows > 0) mbar_arrive_expect_tx(sfull + sb, kStepBytes);", "")],
    # wide-row cluster kernel: clusters of 4 first (n = 32768 -> 32 KiB slices, lagged form, 132 blocks)
    "wide_c4": [("    int order[4] = {8, 2, 4, 16};", "    int order[4] = {4, 8, 2, 16};")],
    # the cluster kernel also for 8192 < n <= 16384 (C = 2 slices of up to 2048 float4), instead of
    # the single-block kernel (timing only: tools/atax_wide_probe.py with WIDE_SHAPES)
    "wide_mid": [("    if (n <= 0 || n % 4 != 0 || fused_plan(n, &narrow)) return false;  // the single-block kernel covers it",
                  "    if (n <= 0 || n % 4 != 0 || n <= 8192) return false;"),
                 ("    if (!fused_plan(n, &p, tune)) {", "    WidePlan w0;\n    if (!fused_plan(n, &p, tune) || (n > 8192 && wide_plan(n, &w0, tune))) {")],
    # the wide kernel without a cluster (C = 1) for 8192 < n <= 16384 instead of the single-block
    # kernel: x, y in registers, rows re-read from the ring one step late
    "wide_c1": [("    if (n <= 0 || n % 4 != 0 || fused_plan(n, &narrow)) return false;  // the single-block kernel covers it",
                 "    if (n <= 0 || n % 4 != 0 || n <= 8192) return false;"),
                ("    for (int c = 2; c <= kFusedMaxCluster; c *= 2) {\n        if (n % (4 * c) != 0) continue;  // every slice",
                 "    for (int c = 1; c <= kFusedMaxCluster; c *= 2) {\n        if (n % (4 * c) != 0) continue;  // every slice"),
                ("    if (!fused_plan(n, &p, tune)) {", "    WidePlan w0;\n    if (!fused_plan(n, &p, tune) || (n > 8192 && wide_plan(n, &w0, tune))) {"),
                ("        if (w.clu == 2) return run_wide<2>(d, w, m, n, A, x, P, y, gbar, s);",
                 "        if (w.clu == 1) return run_wide<1>(d, w, m, n, A, x, P, y, gbar, s);\n        if (w.clu == 2) return run_wide<2>(d, w, m, n, A, x, P, y, gbar, s);"),
                ("            constexpr int VPL = SB / 32;", "            constexpr int VPL = SB >= 32 ? SB / 32 : 1;"),
                ("            for (int u = 0; u < VPL; ++u) v[u] = pb[u];",
                 "            for (int u = 0; u < VPL; ++u) v[u] = (lane * VPL + u < SB) ? pb[u] : 0.f;")],
    # the no-cluster wide kernel down to n > 4096 (8192: threads own 4 of their 8 float4 columns)
    "wide_c1_8k": [("constexpr int64_t kWideMinN = 8192;", "constexpr int64_t kWideMinN = 4096;"),
                   ("        if (nvs <= 4 * (int64_t)kFusedThreads) return false;  // not reached for n > kWideMinN",
                    "        if (nvs <= 2 * (int64_t)kFusedThreads) return false;")],
    # 16 KiB stages (more, smaller bulk copies; twice the steps)
    "stage16": [("constexpr size_t kFusedStageTarget = 32 * 1024;", "constexpr size_t kFusedStageTarget = 16 * 1024;")],
}


def patched(name):
    d = f"/tmp/atax_var_{name}"
    shutil.rmtree(d, ignore_errors=True)
    os.makedirs(d)
    for sub in ("paper_conf_cgo_steuwerrd17_b200", "include", "synth", "oracle", "tools"):
        shutil.copytree(os.path.join(ROOT, sub), os.path.join(d, sub),
                        ignore=shutil.ignore_patterns("_build", "*.so", "__pycache__"))
    shutil.copy(os.path.join(ROOT, "__graft_entry__.py"), d)
    src = open(SRC).read()
    for old, new in VARIANTS[name]:
        assert old in src, (name, old)
        src = src.replace(old, new)
    open(os.path.join(d, "paper_conf_cgo_steuwerrd17_b200", "csrc", "atax.cu"), "w").write(src)
    subprocess.run([sys.executable, "-c", "import __graft_entry__ as g; g.build()"], cwd=d, check=True)
    return d


TIMER = "ab_atax.py"
if "--colpass" in sys.argv:
    sys.argv.remove("--colpass")
    TIMER = "ab_colpass.py"
if "--wide" in sys.argv:  # timing only (tools/atax_wide_probe.py), no bitwise comparison
    sys.argv.remove("--wide")
    TIMER = "atax_wide_probe.py"
names = sys.argv[1:] or list(VARIANTS)
res = {}
for name in names:
    d = patched(name)
    print(f"== {name}", flush=True)
    out = os.path.join(d, "out.npz")
    subprocess.run([sys.executable, os.path.join(ROOT, "tools", TIMER), out], cwd=d, check=True)
    if TIMER != "atax_wide_probe.py":
        res[name] = np.load(out)
if "lib" in res:
    for name, r in res.items():
        same = [k for k in r.files if not k.startswith("t_") and np.array_equal(r[k], res["lib"][k])]
        print(name, "bitwise equal to lib at:", ", ".join(s[2:] for s in same))
