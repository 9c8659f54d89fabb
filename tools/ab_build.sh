#!/bin/bash
# A/B of compile-time variants: for each "TAG=FLAGS" build librj with
# RJ_NVCC_EXTRA=FLAGS and take per-config bench lines.
#   tools/ab_build.sh "base=" "seq=-DRJ_SEQ_SUM" -- C3 C4 C3:accurate
mkdir -p gpurun_out
vars=(); while [ "$1" != "--" ]; do vars+=("$1"); shift; done; shift
for v in "${vars[@]}"; do
  t=${v%%=*}; f=${v#*=}
  RJ_NVCC_EXTRA="$f" python -c "from paper_journals_pvldb_zacharatoudasf17_b200 import _build as b; b.build(force=True)" > gpurun_out/build_ab_$t.log 2>&1 || { echo "build $t failed"; tail gpurun_out/build_ab_$t.log; continue; }
  echo "== $t ($f)"; tools/perf_quick.sh ab_$t "$@" 2>&1 | tail -n +1
done
