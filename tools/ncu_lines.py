"""Per-source-line hot spots of an ncu report (compiled with -lineinfo):
stall samples and executed warp instructions aggregated per CUDA source line.

    python tools/ncu_lines.py report.ncu-rep [top]
"""
import collections
import csv
import io
import subprocess
import sys

rep = sys.argv[1]
top = int(sys.argv[2]) if len(sys.argv) > 2 else 40
kf = ["-k", "regex:" + sys.argv[3], "-c", "1"] if len(sys.argv) > 3 else ["-c", "1"]
out = subprocess.run(["ncu", "-i", rep, *kf, "--page", "source", "--csv", "--print-source=cuda,sass"],
                     capture_output=True, text=True).stdout
rows = list(csv.reader(io.StringIO(out)))
stall = collections.Counter()
inst = collections.Counter()
text = {}
f = "?"
hdr = None
cur = None
for r in rows:
    if len(r) == 2 and r[0] == "File Path":
        f = r[1].split("/")[-1]
        continue
    if r and r[0] == "Line No":
        hdr = {k: i for i, k in enumerate(r)}
        continue
    if hdr is None or len(r) < 5:
        continue
    if r[0]:                       # a CUDA source line (its SASS rows follow with an empty line column)
        cur = (f, int(r[0]))
        text[cur] = r[1].strip()
        continue
    if cur is None:
        continue
    try:
        s = float(r[4] or 0)
        n = float(r[7] or 0)
    except ValueError:
        continue
    stall[cur] += s
    inst[cur] += n
ts = sum(stall.values()) or 1.0
ti = sum(inst.values()) or 1.0
print(f"total stall samples {ts:.0f}, warp instructions {ti:.4g}")
for k, v in stall.most_common(top):
    print(f"{v / ts * 100:5.1f}% stall {inst[k] / ti * 100:5.1f}% inst  {k[0]}:{k[1]}  {text.get(k, '')[:100]}")
