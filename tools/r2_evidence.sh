#!/bin/bash
# Round-2 evidence in GPU calls (profiles/r2_* come from these files).
#   tools/r2_evidence.sh TAG [SECTIONS]   SECTIONS (default all) from:
#   test   GPU tests + smoke
#   bench  contract bench line (+ north-star C4 2B record), reference arm,
#          per-config lines
#   ncu    ncu launch list + full capture of the C2 point pass
#   san    compute-sanitizer (4 tools)
#   emul   strong-scaling emulation
#   full   full-size oracle parity of every config
tag=${1:-r2}; secs=${2:-"test bench ncu san emul full"}
has() { [[ " $secs " == *" $1 "* ]]; }
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_$tag.log 2>&1 || { echo build failed; tail gpurun_out/build_$tag.log; exit 1; }
if has test; then
timeout 1500 python -m pytest tests -m gpu -q -p no:cacheprovider > gpurun_out/pytest_gpu_$tag.log 2>&1; echo "pytest rc=$?"; tail -2 gpurun_out/pytest_gpu_$tag.log
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/smoke_$tag.log 2>&1; echo "smoke rc=$?"; tail -1 gpurun_out/smoke_$tag.log
fi
if has bench; then
timeout 900 python bench.py --ns-c4 > gpurun_out/bench_$tag.json 2> gpurun_out/bench_$tag.err; echo "bench rc=$?"
timeout 300 python bench.py --impl reference --steps 3 --warmup 3 > gpurun_out/bench_ref_$tag.json 2>&1; echo "ref rc=$?"
tools/perf_quick.sh cfg_$tag C2 C3:bounded C3:accurate C3:index C4 C5 C5:accurate > gpurun_out/cfg_$tag.txt 2>&1; cat gpurun_out/cfg_$tag.txt
fi
if has ncu; then
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none -c 600 --csv --log-file /tmp/launches_$tag.csv \
   python bench.py --steps 3 --warmup 3 --e2e-steps 0 --no-cpu-baseline > /dev/null 2>&1; echo "ncu list rc=$?"
python tools/ncu_summary.py --launches /tmp/launches_$tag.csv 6 > gpurun_out/launches_C2_$tag.md 2>&1
timeout 900 ncu --set full --clock-control none --import-source on -k regex:k_point_pass -s 2 -c 1 -o /tmp/prof_C2_$tag -f \
   python bench.py --steps 1 --warmup 3 --e2e-steps 0 --no-cpu-baseline > /dev/null 2>&1; echo "ncu full rc=$?"
cp /tmp/prof_C2_$tag.ncu-rep gpurun_out/ 2>/dev/null
python tools/ncu_summary.py /tmp/prof_C2_$tag.ncu-rep > gpurun_out/ncu_C2_$tag.md 2>&1
python tools/ncu_lines.py /tmp/prof_C2_$tag.ncu-rep 30 > gpurun_out/ncu_C2_lines_$tag.txt 2>&1
fi
if has san; then
SAN_TIMEOUT=900 tools/sanitize.sh $tag > gpurun_out/sanitize_$tag.log 2>&1; grep "rc=" gpurun_out/sanitize_$tag.log
fi
if has emul; then
for cfg in "C4 --points 2e9" "C2 --points 1e9" "C3 --points 1e9"; do
  timeout 900 python tools/emulate_strong.py --config $cfg --ranks 2,4,8 --spatial-only --poly-weight 0.1 >> gpurun_out/emul_$tag.jsonl 2>>gpurun_out/emul_$tag.err
done; echo "emul done"
fi
if has full; then
timeout 3000 python tools/fullsize_parity.py --out gpurun_out/fullsize_parity_$tag.jsonl > gpurun_out/fullsize_$tag.log 2>&1; echo "fullsize rc=$?"
fi
