#!/bin/bash
# Quick per-config bench lines (no cpu baseline, no e2e): TAG CFG:MODE ...
tag=$1; shift
mkdir -p gpurun_out
: > gpurun_out/perf_$tag.jsonl
for spec in "$@"; do
  flags=""; case "$spec" in *+*) flags="${spec#*+}"; spec="${spec%%+*}"; flags="--${flags//+/ --}";; esac
  cfg=${spec%%:*}; mode=${spec#*:}
  extra="$flags"; [ "$mode" != "$cfg" ] && extra="$extra --mode $mode"
  timeout 600 python bench.py --config $cfg $extra --steps 10 --warmup 3 --no-cpu-baseline --e2e-steps 0 \
     2> gpurun_out/perf_${tag}_${cfg}_${mode}.err | tail -1 >> gpurun_out/perf_$tag.jsonl
done
python tools/bench_table.py gpurun_out/perf_$tag.jsonl 2>/dev/null || cat gpurun_out/perf_$tag.jsonl
