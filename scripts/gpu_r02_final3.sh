# the round's final evidence: scripts/gpu_r02_final.sh + the torchrun launch path at N = 1
TAG=${1:-r02_final3}
bash scripts/gpu_r02_final.sh $TAG
OUT=gpurun_out/$TAG
timeout 600 python -m torch.distributed.run --nnodes=1 --nproc-per-node 1 --master-addr 127.0.0.1 --master-port 29533 \
  bench.py --gpus 1 --steps 3 --warmup 3 --no-cpu-baseline --no-extras > $OUT/bench_torchrun1.log 2>&1
echo "TORCHRUN rc=$? $(tail -1 $OUT/bench_torchrun1.log | cut -c1-160)"
python scripts/dev/e2e_breakdown.py csp > $OUT/e2e_breakdown.json 2> $OUT/e2e_breakdown.err; tail -1 $OUT/e2e_breakdown.json
