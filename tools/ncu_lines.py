"""Per-source-line warp-stall summary of an ncu report (tuning aid).

usage: python tools/ncu_lines.py REPORT.ncu-rep [top]
Runs `ncu -i REPORT --page source --csv --print-source=cuda,sass`, attributes every
SASS instruction's stall samples to the CUDA source line above it, and prints the
top lines with their dominant stall reasons.
"""
import collections
import csv
import io
import subprocess
import sys

rep = sys.argv[1]
top = int(sys.argv[2]) if len(sys.argv) > 2 else 25
out = subprocess.run(["ncu", "-i", rep, "--page", "source", "--csv", "--print-source=cuda,sass"],
                     capture_output=True, text=True).stdout
rows = list(csv.reader(io.StringIO(out)))
hdr_i = next(i for i, r in enumerate(rows) if r[:2] == ["Line No", "Source"])
hdr = rows[hdr_i]
col = {h: i for i, h in enumerate(hdr) if i >= 4}
samp = col["Warp Stall Sampling (All Samples)"]
stalls = [h for h in hdr[4:] if h.startswith("stall_") and "Not Issued" not in h]
per_line = collections.OrderedDict()
line, text, total = None, "", 0
file_name = ""
for r in rows[hdr_i + 1:]:
    if r and r[0] == "File Path":
        file_name = r[1].rsplit("/", 1)[-1]
        continue
    if len(r) < len(hdr):
        continue
    if r[0] not in ("", "-"):
        line, text = f"{file_name}:{r[0]}", r[1]
        continue
    try:
        s = int(r[samp] or 0)
    except ValueError:
        continue
    if not s:
        continue
    total += s
    d = per_line.setdefault(line, {"text": text, "n": 0, "st": collections.Counter()})
    d["n"] += s
    for h in stalls:
        try:
            v = int(r[hdr.index(h, 4)] or 0)
        except ValueError:
            v = 0
        if v:
            d["st"][h[6:]] += v
print(f"{total} samples")
for ln, d in sorted(per_line.items(), key=lambda t: -t[1]["n"])[:top]:
    st = ", ".join(f"{k} {v}" for k, v in d["st"].most_common(3))
    print(f"{d['n']:6d} {100 * d['n'] / total:5.1f}%  {ln:18s} {d['text'].strip()[:70]:70s} [{st}]")
