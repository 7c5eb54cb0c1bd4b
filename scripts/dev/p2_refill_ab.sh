# A/B ab14 (rejected, profiles/ab/r01_ab14_phase2_refill.md): needs the temporary NT_DEV_P2_REFILL hook
# in track_phases (nt_api.cu) that set phase 2 refill_min; the hook was removed after the A/B.
mkdir -p gpurun_out/p2
for rep in 1 2; do
 for c in csp split; do
  for v in 4 1 2 8 16; do
   NT_DEV_P2_REFILL=$v python bench.py --config $c --no-cpu-baseline --no-e2e --steps 5 --json-out gpurun_out/p2/${c}_${v}_$rep.json > /dev/null 2>&1
   python -c "import json,sys; d=json.load(open(sys.argv[1])); print(sys.argv[1], round(d['roofline']['kernel_ms'],3))" gpurun_out/p2/${c}_${v}_$rep.json
  done
 done
done
