#!/bin/bash
# One GPU call for an iteration: build, selected tests, bench lines, optional ncu capture.
#   tools/gpu_iter.sh TAG "pytest args" "CFG:MODE[:extra bench args] ..." [NCU_CFG[:MODE]]
tag=$1; tests=$2; benches=$3; ncucfg=$4
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_$tag.log 2>&1 || { echo build failed; tail -20 gpurun_out/build_$tag.log; exit 1; }
if [ -n "$tests" ]; then
  timeout 1500 python -m pytest $tests -q -x > gpurun_out/pytest_$tag.log 2>&1; echo "pytest rc=$?"; tail -5 gpurun_out/pytest_$tag.log
fi
: > gpurun_out/bench_$tag.jsonl
for spec in $benches; do
  IFS=: read cfg mode extra <<< "$spec"
  args="--config $cfg"; [ -n "$mode" ] && args="$args --mode $mode"
  [ -n "$extra" ] && args="$args ${extra//,/ }"
  timeout 600 python bench.py $args --steps 10 --warmup 3 --no-cpu-baseline --e2e-steps 0 2> gpurun_out/bench_${tag}_${cfg}_${mode}.err | tail -1 >> gpurun_out/bench_$tag.jsonl
done
python tools/bench_table.py gpurun_out/bench_$tag.jsonl
for spec in $ncucfg; do
  IFS=: read cfg mode extra <<< "$spec"
  args="--config $cfg"; [ -n "$mode" ] && args="$args --mode $mode"
  [ -n "$extra" ] && args="$args ${extra//,/ }"
  name=$(echo "${cfg}_${mode}_${extra}" | tr -c 'A-Za-z0-9_\n' '_')
  timeout 900 ncu --set full --clock-control none --import-source on -k regex:"k_point_pass|k_pip_queue" -s 2 -c 2 -o gpurun_out/prof_${name}_$tag -f \
     python bench.py $args --steps 1 --warmup 3 --e2e-steps 0 --no-cpu-baseline > gpurun_out/ncu_${name}_$tag.log 2>&1; echo "ncu $name rc=$?"
done
