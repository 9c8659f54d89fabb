"""Print one line per bench JSON line: config, points/s, step ms, kernel ms, roofline fraction, stages."""
import json
import sys

for l in open(sys.argv[1]):
    l = l.strip()
    if not l.startswith("{"):
        continue
    d = json.loads(l)
    r = d["roofline"]
    print(f"{d['config']['workload'][:70]:70s} {d['value'] / 1e9:8.1f} G/s  step {d['ms_per_step']:7.3f}  "
          f"kern {r['kernel_ms']:7.3f}  frac {r['frac']:.3f}  poly {d['stages_ms']['polygon_pass']:.3f}  "
          f"nb {d['checks']['n_boundary']}  {d['launch']}")
