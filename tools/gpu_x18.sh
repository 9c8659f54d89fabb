mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > /dev/null 2>&1
for w in 0.0 0.05 0.1 0.2; do
  echo "C4 w=$w"; timeout 600 python tools/emulate_strong.py --config C4 --points 2e9 --ranks 4,8 --spatial-only --poly-weight $w 2>/dev/null | head -2 | cut -c1-200
done
for w in 0.0 0.1 0.2; do
  echo "C3 w=$w"; timeout 600 python tools/emulate_strong.py --config C3 --ranks 8 --spatial-only --poly-weight $w 2>/dev/null | head -1 | cut -c1-200
done
