"""Turn a GPU session's ncu output (gpurun_out/<tag>/) into committed summaries under profiles/.

    python tools/make_profiles.py <tag> <round-prefix>

Writes profiles/<prefix>_launches.csv (raw launch list of the bench command),
profiles/<prefix>_launches.txt (per-launch table + per-kernel share of the
step), profiles/<prefix>_ncu_full_<name>.txt (key metrics of each --set full
capture) and updates profiles/traffic.json (DRAM bytes per launch from the
full captures, used by bench.py's roofline.traffic).
"""
import collections
import csv
import io
import json
import os
import shutil
import subprocess
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, os.path.join(ROOT, "tools"))
from ncu_summary import load  # noqa: E402

KEY = ["Duration", "Elapsed Cycles", "SM Active Cycles", "SM Frequency", "DRAM Frequency", "DRAM Throughput",
       "Memory Throughput", "L2 Hit Rate", "Registers Per Thread", "Block Size", "Grid Size", "Theoretical Occupancy",
       "Achieved Occupancy", "Issue Slots Busy", "Executed Instructions", "No Eligible",
       "Warp Cycles Per Issued Instruction", "Dynamic Shared Memory Per Block", "Waves Per SM"]
RAW = ["dram__bytes_read.sum", "dram__bytes_write.sum", "gpu__time_duration.sum", "lts__t_bytes.sum",
       "sm__throughput.avg.pct_of_peak_sustained_elapsed", "gpu__dram_throughput.avg.pct_of_peak_sustained_elapsed"]


def ncu_csv(rep, page):
    return subprocess.run(["ncu", "-i", rep, "--page", page, "--csv"], capture_output=True, text=True).stdout


def full_summary(rep):
    out = []
    det = list(csv.reader(io.StringIO(ncu_csv(rep, "details"))))
    h = det[0]
    name = None
    for row in det[1:]:
        d = dict(zip(h, row))
        name = d.get("Kernel Name", name)
        if d.get("Metric Name") in KEY:
            out.append(f"{d['Metric Name']:40s} {d['Metric Unit']:>14s} {d['Metric Value']}")
    raw = list(csv.reader(io.StringIO(ncu_csv(rep, "raw"))))
    vals = {}
    if len(raw) >= 3:
        for n, u, v in zip(raw[0], raw[1], raw[2]):
            if n in RAW:
                vals[n] = (u, v)
        stalls = []
        for n, u, v in zip(raw[0], raw[1], raw[2]):
            if n.startswith("smsp__pcsamp_warps_issue_stalled_") and not n.endswith("_not_issued"):
                try:
                    stalls.append((float(v.replace(",", "")), n.replace("smsp__pcsamp_warps_issue_stalled_", "")))
                except ValueError:
                    pass
        stalls.sort(reverse=True)
    else:
        stalls = []
    for n in RAW:
        if n in vals:
            out.append(f"{n:40s} {vals[n][0]:>14s} {vals[n][1]}")
    if stalls:
        tot = sum(s for s, _ in stalls) or 1
        out.append("top stall reasons (pc sampling): " + ", ".join(f"{n} {100 * s / tot:.0f}%" for s, n in stalls[:6]))
    return name, out, vals


def main(tag, prefix):
    src = os.path.join(ROOT, "gpurun_out", tag)
    dst = os.path.join(ROOT, "profiles")
    os.makedirs(dst, exist_ok=True)
    lc = os.path.join(src, "launches.csv")
    if os.path.exists(lc):
        shutil.copy(lc, os.path.join(dst, f"{prefix}_launches.csv"))
        k = load(lc)
        lines = [f"# ncu launch list of `python bench.py --steps 2 --warmup 3 --no-e2e --no-cpu` ({tag});",
                 "# cold-cache, serialised per-launch times: compare SHARES of the step, not absolutes", ""]
        tot = collections.OrderedDict()
        # bench.py --steps 2 --warmup 3 launches: 3 eager warm-up steps, then the CUDA graph of
        # the 2 timed steps replayed twice (upload, then timed), then the per-op breakdown
        kps, warm, steps = 5, 3, 2
        t0, t1 = (warm + steps) * kps, (warm + 2 * steps) * kps
        for i, d in k.items():
            t = d.get("gpu__time_duration.sum", 0.0)
            rd, wr = d.get("dram__bytes_read.sum", 0.0), d.get("dram__bytes_write.sum", 0.0)
            nm = d["name"].split("(")[0].replace("void ", "")
            lines.append(f"{i:>4} {nm:34s} grid {d['grid']:>14} {t / 1e3:10.2f} us  dram {(rd + wr) / 1e6:10.2f} MB"
                         f"  {(rd + wr) / t if t else 0:8.1f} GB/s")
            if t0 <= int(i) < t1:  # the timed steps only
                a = tot.setdefault(nm, [0.0, 0.0, 0])
                a[0] += t
                a[1] += rd + wr
                a[2] += 1
        s = sum(v[0] for v in tot.values()) or 1
        lines += ["", f"per-kernel share of the timed steps (launches {t0}..{t1 - 1}, ncu time):"]
        for nm, (t, b, c) in sorted(tot.items(), key=lambda kv: -kv[1][0]):
            lines.append(f"  {nm:34s} launches {c:3d}  share {100 * t / s:6.2f}%  avg {t / c / 1e3:10.2f} us  "
                         f"dram/launch {b / c / 1e6:10.2f} MB")
        open(os.path.join(dst, f"{prefix}_launches.txt"), "w").write("\n".join(lines) + "\n")
    tj = os.path.join(dst, "traffic.json")
    traffic = json.load(open(tj)) if os.path.exists(tj) else {}
    traffic = {k: v for k, v in traffic.items() if ":" in k}
    for f in sorted(os.listdir(src)):
        if f.startswith("full_") and f.endswith(".ncu-rep"):
            label = f[len("full_"):-len(".ncu-rep")]
            name, out, vals = full_summary(os.path.join(src, f))
            hdr = [f"# ncu --set full --clock-control none --import-source on; {tag}/{f}", f"# kernel: {name}", ""]
            open(os.path.join(dst, f"{prefix}_ncu_full_{label}.txt"), "w").write("\n".join(hdr + out) + "\n")
            if "dram__bytes_read.sum" in vals and name:
                def num(x):
                    return float(x[1].replace(",", ""))

                unit = {"byte": 1, "Kbyte": 1e3, "Mbyte": 1e6, "Gbyte": 1e9}
                b = num(vals["dram__bytes_read.sum"]) * unit.get(vals["dram__bytes_read.sum"][0], 1) + \
                    num(vals["dram__bytes_write.sum"]) * unit.get(vals["dram__bytes_write.sum"][0], 1)
                kern = name.split("(")[0].replace("void ", "").split("<")[0].strip()
                ent = {"dram_bytes_per_launch": b, "source": f"profiles/{prefix}_ncu_full_{label}.txt"}
                pct = vals.get("gpu__dram_throughput.avg.pct_of_peak_sustained_elapsed")
                if pct is not None:
                    ent["ncu_dram_pct_of_peak"] = round(float(pct[1].replace(",", "")), 2)
                dur = vals.get("gpu__time_duration.sum")
                if dur is not None:
                    scale = {"ns": 1e-3, "usecond": 1.0, "us": 1.0, "ms": 1e3, "msecond": 1e3}.get(dur[0], 1.0)
                    ent["ncu_duration_us"] = round(float(dur[1].replace(",", "")) * scale, 3)
                traffic[kern + ":" + label] = ent
    json.dump(traffic, open(tj, "w"), indent=1, sort_keys=True)
    table1(src, dst, tag, prefix)


def table1(src, dst, tag, prefix, calls=4):
    """ncu launch lists of tools/table1.py NAME (4 calls on distinct operands each)
    -> profiles/table1_ncu.json (read by bench.py) + profiles/<prefix>_table1_ncu.txt."""
    files = sorted(f for f in os.listdir(src) if f.startswith("table1_") and f.endswith(".csv"))
    if not files:
        return
    res, lines = {}, [f"# ncu --metrics gpu__time_duration.sum,dram__bytes_*.sum,gpu__dram_throughput.avg."
                      f"pct_of_peak_sustained_elapsed --clock-control none ({tag}): tools/table1.py NAME,",
                      "# 4 calls on distinct operands, cold L2 (ncu flushes before every launch); per call: "
                      "summed kernel time, DRAM bytes, time-weighted DRAM % of peak; median over the calls", ""]
    for f in files:
        name = f[len("table1_"):-len(".csv")]
        try:
            k = list(load(os.path.join(src, f)).values())
        except StopIteration:
            continue
        if not k or len(k) % calls:
            continue
        per = len(k) // calls
        rows = []
        for c in range(calls):
            ks = k[c * per:(c + 1) * per]
            t = sum(d.get("gpu__time_duration.sum", 0.0) for d in ks)
            b = sum(d.get("dram__bytes_read.sum", 0.0) + d.get("dram__bytes_write.sum", 0.0) for d in ks)
            pct = sum(d.get("gpu__dram_throughput.avg.pct_of_peak_sustained_elapsed", 0.0) *
                      d.get("gpu__time_duration.sum", 0.0) for d in ks) / (t or 1)
            rows.append((t, b, pct))
        rows.sort()
        t, b, pct = rows[len(rows) // 2]
        res[name] = {"us": round(t / 1e3, 2), "dram_bytes": b, "ncu_dram_pct_of_peak": round(pct, 2),
                     "kernels_per_call": per}
        names = ", ".join(sorted({d["name"].split("(")[0].replace("void ", "").split("<")[0] for d in k}))
        lines.append(f"{name:26s} {t / 1e3:9.2f} us  dram {b / 1e6:9.2f} MB  {b / t if t else 0:8.1f} GB/s  "
                     f"DRAM {pct:6.2f}% of peak  ({per} kernel(s)/call: {names})")
    json.dump(res, open(os.path.join(dst, "table1_ncu.json"), "w"), indent=1, sort_keys=True)
    open(os.path.join(dst, f"{prefix}_table1_ncu.txt"), "w").write("\n".join(lines) + "\n")


if __name__ == "__main__":
    main(sys.argv[1], sys.argv[2])
