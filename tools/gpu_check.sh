#!/bin/bash
# One GPU call: full GPU test suite + smoke + a few bench lines (args: extra bench runs "CFG:MODE ...").
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build.log 2>&1
timeout 1500 python -m pytest tests -m gpu -q -x > gpurun_out/pytest_gpu.log 2>&1; echo "pytest rc=$?" >> gpurun_out/pytest_gpu.log
timeout 300 python -c "import __graft_entry__ as g; g.smoke(); print('smoke ok')" > gpurun_out/smoke.log 2>&1
: > gpurun_out/bench_lines.jsonl
for spec in "$@"; do
  cfg=${spec%%:*}; mode=${spec#*:}
  extra=""; [ "$mode" != "$cfg" ] && extra="--mode $mode"
  timeout 600 python bench.py --config $cfg $extra --steps 10 --warmup 3 --no-cpu-baseline --e2e-steps 1 \
     2> gpurun_out/bench_${cfg}_${mode}.err | tail -1 >> gpurun_out/bench_lines.jsonl
done
