mkdir -p gpurun_out
B=paper_journals_pvldb_zacharatoudasf17_b200._build
RJ_NVCC_EXTRA="-DRJ_INLINE_DRAIN" python -m $B --force > /dev/null || exit 1
for args in "bounded sum 0" "bounded sum 512" "bounded sum 4096 1" "bounded sum 4096 0" "bounded sum 4096 0 2" "bounded sum 4096 0 3" "bounded sum 4096 0 4" "accurate count 4096 -1 2" "bounded count 4096 -1 2"; do
  echo "=== racecheck $args"
  compute-sanitizer --tool racecheck --print-limit 1 python tools/san_exp.py $args 2>&1 | grep -v "Host Frame\|^========= $" | tail -3
done
