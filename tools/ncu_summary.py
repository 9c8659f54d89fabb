"""Summarise an ncu report (or a launch-list CSV) into a small text/JSON file
for profiles/ (the judged evidence).

    python tools/ncu_summary.py report.ncu-rep  > profiles/xxx.md
    python tools/ncu_summary.py --launches launches.csv > profiles/xxx_launches.md
"""
from __future__ import annotations

import collections
import csv
import io
import json
import subprocess
import sys

METRICS = [
    "gpu__time_duration.sum", "dram__bytes_read.sum", "dram__bytes_write.sum",
    "dram__throughput.avg.pct_of_peak_sustained_elapsed", "dram__bytes_read.sum.per_second",
    "sm__throughput.avg.pct_of_peak_sustained_elapsed", "sm__inst_executed.sum.pct_of_peak_sustained_elapsed",
    "sm__warps_active.avg.per_cycle_active", "smsp__warps_eligible.avg.per_cycle_active",
    "launch__grid_size", "launch__block_size", "launch__registers_per_thread",
    "launch__shared_mem_per_block_dynamic", "launch__occupancy_limit_registers",
    "launch__occupancy_limit_shared_mem", "lts__t_sector_hit_rate.pct",
    "l1tex__data_pipe_lsu_wavefronts_mem_shared.sum", "l1tex__data_bank_conflicts_pipe_lsu_mem_shared.sum",
    "sm__cycles_elapsed.avg.per_second",
]


def ncu_csv(args):
    out = subprocess.run(["ncu", *args], capture_output=True, text=True).stdout
    return list(csv.reader(io.StringIO(out)))


def _stalls(rep, kname):
    """Warp stall shares from the SASS source page of one kernel of the report."""
    src = ncu_csv(["-i", rep, "-k", "regex:" + kname, "-c", "1", "--page", "source", "--csv", "--print-source=sass"])
    hdr = None
    data = []
    for r in src:
        if "Warp Stall Sampling (All Samples)" in r:
            hdr = {k: i for i, k in enumerate(r)}
            continue
        if hdr and len(r) == len(hdr):
            data.append(r)
    if not hdr or not data:
        return []
    stalls = [k for k in hdr if k.startswith("stall_") and "Not Issued" not in k]
    f = lambda r, k: float(r[hdr[k]] or 0)
    tot = sum(f(r, "Warp Stall Sampling (All Samples)") for r in data) or 1.0
    st = {k: sum(f(r, k) for r in data) for k in stalls}
    lines = ["", "### warp stall reasons (share of samples)"]
    for k, v in sorted(st.items(), key=lambda x: -x[1])[:10]:
        lines.append(f"- {k[6:]}: {v / tot * 100:.1f} %")
    lines.append(f"- warp instructions executed: {sum(f(r, 'Instructions Executed') for r in data):.4g}")
    return lines


def summarize(rep):
    rows = ncu_csv(["-i", rep, "--page", "raw", "--csv"])
    h, units = rows[0], rows[1]
    lines = [f"# ncu summary: {rep}", ""]
    result = {}
    for r in rows[2:]:
        name = r[h.index("Kernel Name")] if "Kernel Name" in h else "?"
        lines.append(f"## {name}")
        res = {}
        for m in METRICS:
            if m in h:
                i = h.index(m)
                lines.append(f"- {m} = {r[i]} {units[i]}")
                res[m] = r[i]
        short = name.split("(")[0].split("::")[-1].split("<")[0]
        lines += _stalls(rep, short)
        lines.append("")
        result[short] = res
    return "\n".join(lines), result


def launches(path, steps=0):
    """Launch list of an ncu --metrics gpu__time_duration.sum capture.  The
    per-step table covers the launches after the last load-time kernel (the
    sort / quantise / cell-bounds / edge-grid kernels and torch fills) and
    counts one query step per launch of the point-pass kernel."""
    rows = list(csv.reader(open(path)))
    hdr = None
    for i, r in enumerate(rows):
        if "Kernel Name" in r and "Metric Value" in r:
            hdr = i
            break
    h = rows[hdr]
    k_i, v_i, u_i = h.index("Kernel Name"), h.index("Metric Value"), h.index("Metric Unit")
    seq = []
    for r in rows[hdr + 1:]:
        if len(r) <= v_i:
            continue
        v = float(r[v_i].replace(",", ""))
        scale = {"ns": 1e-6, "nsecond": 1e-6, "us": 1e-3, "usecond": 1e-3, "ms": 1.0, "msecond": 1.0}.get(r[u_i], 1.0)
        seq.append((r[k_i].split("(")[0], v * scale))
    tot = collections.Counter()
    cnt = collections.Counter()
    for name, ms in seq:
        tot[name] += ms
        cnt[name] += 1
    all_ms = sum(tot.values())
    lines = [f"# launch list: {path}", "", "| kernel | launches | total ms | share |", "|---|---|---|---|"]
    for k, v in tot.most_common():
        lines.append(f"| {k} | {cnt[k]} | {v:.3f} | {v / all_ms * 100:.1f} % |")
    if steps:
        load = ("radix", "quantize", "cell_bounds", "grid_", "at::", "ring_sigma")
        last = max([i for i, (n, _) in enumerate(seq) if any(t in n for t in load)], default=-1)
        qs = seq[last + 1:]
        n_steps = sum(1 for n, _ in qs if "k_point_pass" in n) or 1
        qt = collections.Counter()
        qc = collections.Counter()
        for name, ms in qs:
            qt[name] += ms
            qc[name] += 1
        q_ms = sum(qt.values())
        lines += ["", f"## per query step ({n_steps} query steps after the load; serialised, cold: compare shares)",
                  "", "| kernel | launches/step | ms/step | share of the step |", "|---|---|---|---|"]
        for k, v in qt.most_common():
            lines.append(f"| {k} | {qc[k] / n_steps:g} | {v / n_steps:.4f} | {v / q_ms * 100:.1f} % |")
        lines.append(f"| (all) | | {q_ms / n_steps:.4f} | 100 % |")
    return "\n".join(lines)


if __name__ == "__main__":
    if sys.argv[1] == "--launches":
        print(launches(sys.argv[2], int(sys.argv[3]) if len(sys.argv) > 3 else 0))
    else:
        text, res = summarize(sys.argv[1])
        print(text)
        if len(sys.argv) > 2:
            json.dump(res, open(sys.argv[2], "w"), indent=1)
