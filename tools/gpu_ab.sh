#!/bin/bash
# One GPU call for a kernel change: build, full GPU suite, then bench lines
# of the given configs.  Usage: tools/gpu_ab.sh TAG CFG:MODE ...
tag=${1:-ab}; shift
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_$tag.log 2>&1 || { echo build failed; tail gpurun_out/build_$tag.log; exit 1; }
timeout 1200 python -m pytest tests -m gpu -q -x > gpurun_out/pytest_gpu_$tag.log 2>&1; echo "pytest rc=$?"; tail -3 gpurun_out/pytest_gpu_$tag.log
: > gpurun_out/bench_lines_$tag.jsonl
for spec in "$@"; do
  cfg=${spec%%:*}; mode=${spec#*:}
  timeout 600 python bench.py --config $cfg --mode $mode --steps 10 --warmup 3 --no-cpu-baseline --e2e-steps 1 \
     2> gpurun_out/bench_${tag}_${cfg}_${mode}.err | tail -1 >> gpurun_out/bench_lines_$tag.jsonl
done
python - "$tag" <<'PY'
import json, sys
for l in open(f"gpurun_out/bench_lines_{sys.argv[1]}.jsonl"):
    d = json.loads(l)
    print(d["config"]["workload"][-45:], round(d["ms_per_step"], 3), {k: round(v, 3) for k, v in d["stages_ms"].items()})
PY
