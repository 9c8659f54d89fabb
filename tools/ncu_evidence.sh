#!/bin/bash
# One ncu call (the guide: at most one profiler tool per gpurun call):
# per-launch lists of C2 / C3 accurate / C5 (--metrics gpu__time_duration,
# serialised, cold) and a full capture of the C2 point pass.  Each command
# runs once without ncu first and must exit 0.   tools/ncu_evidence.sh TAG
tag=${1:-r2}
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_$tag.log 2>&1 || exit 1
B="python bench.py --steps 3 --warmup 3 --e2e-steps 0 --no-cpu-baseline"
for spec in "C2:" "C3a:--config C3" "C5:--config C5" "C5a:--config C5 --mode accurate"; do
  name=${spec%%:*}; args=${spec#*:}
  $B $args > gpurun_out/plain_${name}_$tag.log 2>&1 && \
  timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none -c 800 --csv --log-file gpurun_out/launches_${name}_$tag.csv \
     $B $args > /dev/null 2>&1; echo "list $name rc=$?"
  python tools/ncu_summary.py --launches gpurun_out/launches_${name}_$tag.csv 3 > gpurun_out/launches_${name}_$tag.md 2>&1
done
P="python bench.py --steps 1 --warmup 3 --e2e-steps 0 --no-cpu-baseline"
$P > gpurun_out/plain_full_$tag.log 2>&1 && \
timeout 900 ncu --set full --clock-control none --import-source on -k regex:k_point_pass -s 2 -c 1 -o gpurun_out/prof_C2_$tag -f $P > /dev/null 2>&1; echo "ncu full rc=$?"
python tools/ncu_summary.py gpurun_out/prof_C2_$tag.ncu-rep > gpurun_out/ncu_C2_$tag.md 2>&1
python tools/ncu_lines.py gpurun_out/prof_C2_$tag.ncu-rep 30 > gpurun_out/ncu_C2_lines_$tag.txt 2>&1
