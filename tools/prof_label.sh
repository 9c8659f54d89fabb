#!/bin/bash
# ncu (one tool per call) of the label kernel at C4 and C3 accurate, source lines
tag=${1:-lab}
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_$tag.log 2>&1 || exit 1
for spec in "C4:--config C4" "C3a:--config C3"; do
  name=${spec%%:*}; args=${spec#*:}
  P="python bench.py $args --steps 1 --warmup 3 --e2e-steps 0 --no-cpu-baseline"
  $P > gpurun_out/plain_${name}_$tag.log 2>&1 && \
  timeout 900 ncu --set full --clock-control none --import-source on -k regex:"k_point_pass|k_pip" -s 2 -c 2 -o gpurun_out/prof_${name}_$tag -f $P > /dev/null 2>&1; echo "ncu $name rc=$?"
  python tools/ncu_summary.py gpurun_out/prof_${name}_$tag.ncu-rep > gpurun_out/ncu_${name}_$tag.md 2>&1
  python tools/ncu_lines.py gpurun_out/prof_${name}_$tag.ncu-rep 60 k_point_pass > gpurun_out/lines_${name}_$tag.txt 2>&1
done
