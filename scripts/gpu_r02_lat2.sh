# ncu of a lone-history run (stream, 148 particles: one lane per SM): where a facet's latency goes
OUT=gpurun_out/r02_lat2; mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()"
timeout 600 ncu --set full --clock-control none --import-source on -k regex:history -c 1 -o $OUT/prof_lone \
  python bench.py --config stream --particles 148 --steps 1 --warmup 0 --no-cpu-baseline --no-e2e --no-extras > $OUT/ncu.log 2>&1
python scripts/ncu_summary.py $OUT/prof_lone.ncu-rep $OUT/ncu_lone.md --top 40 > /dev/null 2>&1
ncu -i $OUT/prof_lone.ncu-rep --page source --csv --print-source sass > $OUT/sass_lone.csv 2>/dev/null
rm -f $OUT/prof_lone.ncu-rep
ls -la $OUT
