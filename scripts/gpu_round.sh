# usage: bash scripts/gpu_round.sh TAG -- the round's evidence: GPU tests, default bench (csp, with
# cpu_baseline + e2e), the other configs, launch list, ncu --set full of csp/stream history.
TAG=${1:-round}
OUT=gpurun_out/$TAG
mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()"
timeout 1200 python -m pytest tests -m gpu -x -q -p no:cacheprovider > $OUT/pytest_gpu.log 2>&1
tail -1 $OUT/pytest_gpu.log | sed "s/^/PYTEST: /"
timeout 600 python -c "import __graft_entry__ as g; g.smoke()" > $OUT/smoke.log 2>&1; echo "SMOKE rc=$?: $(tail -1 $OUT/smoke.log)"
timeout 600 python bench.py --impl reference --steps 2 --warmup 1 > $OUT/bench_reference.log 2>&1; echo "REFERENCE: $(tail -1 $OUT/bench_reference.log | cut -c1-200)"
python bench.py --json-out $OUT/bench_csp.json > $OUT/bench_csp.log 2>&1
for c in stream scatter split stream_8m; do
  python bench.py --config $c --no-cpu-baseline --no-e2e --steps 5 --json-out $OUT/bench_$c.json > $OUT/bench_$c.log 2>&1
done
for c in csp stream scatter split; do
  python bench.py --config $c --mode event --no-cpu-baseline --no-e2e --steps 3 --json-out $OUT/bench_${c}_event.json > $OUT/bench_${c}_event.log 2>&1
done
for f in $OUT/bench_*.json; do python -c "
import json; d=json.load(open('$f')); r=d['roofline']
print('$f'.split('/')[-1], f\"value={d['value']:.3e} ms={d['ms_per_step']:.2f} frac={r['frac']:.3f} clocks={d['clocks']['sm_mhz']}\")"; done
ncu --metrics gpu__time_duration.sum --clock-control none -c 400 --csv --log-file $OUT/launches_csp.csv \
    python bench.py --steps 2 --warmup 1 --no-cpu-baseline --no-e2e > $OUT/ncu_launch_bench.log 2>&1
for c in csp stream scatter; do
  ncu --set full --clock-control none --import-source on -k regex:history -s 2 -c 2 \
      -o $OUT/prof_${c} python bench.py --config $c --steps 1 --warmup 1 --no-cpu-baseline --no-e2e > $OUT/ncu_$c.log 2>&1
done
ncu --set full --clock-control none --import-source on -k regex:ev_loop -c 1 \
    -o $OUT/prof_csp_event python bench.py --mode event --steps 1 --warmup 0 --no-cpu-baseline --no-e2e > $OUT/ncu_csp_event.log 2>&1
# summaries on the box (the reports themselves would exceed gpurun's 64 MiB return limit)
for r in csp stream scatter csp_event; do
  k=$(echo $r | sed 's/_event/\/event/; t; s/$/\/history/')
  python scripts/ncu_summary.py $OUT/prof_$r.ncu-rep $OUT/ncu_${r}.md --traffic-key $k > /dev/null 2>&1
done
for r in stream scatter csp_event; do rm -f $OUT/prof_$r.ncu-rep; done
ls $OUT
