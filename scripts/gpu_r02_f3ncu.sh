# ncu --set full pairs for the f3 ablations (tally modes, AoS): phase-1 history launch each
OUT=gpurun_out/r02_f3; mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()"
run() {  # name, bench args
  timeout 900 ncu --set full --clock-control none --import-source on -k regex:history_kernel -c 1 -o $OUT/prof_$1 python bench.py --steps 1 --warmup 0 --no-cpu-baseline --no-e2e --no-extras $2 > $OUT/ncu_$1.log 2>&1
  python scripts/ncu_summary.py $OUT/prof_$1.ncu-rep $OUT/ncu_$1.md > /dev/null 2>&1
  rm -f $OUT/prof_$1.ncu-rep
  grep -E "gpu__time_duration|lts__throughput|issue_active" $OUT/ncu_$1.md | head -3 | sed "s/^/$1 /"
}
run csp_red "--config csp --tally-mode 0"
run csp_cas "--config csp --tally-mode 2"
run src001_red "--config scatter_src001 --tally-mode 0"
run src001_hot "--config scatter_src001 --tally-mode 3"
run src001_warpagg "--config scatter_src001 --tally-mode 1"
run scatter_soa "--config scatter --particle-layout 0"
run scatter_aos "--config scatter --particle-layout 1"
