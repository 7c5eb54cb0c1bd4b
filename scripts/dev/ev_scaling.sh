for n in 1000 30000 300000 1000000; do
  python bench.py --config stream --mode event --particles $n --no-cpu-baseline --no-e2e --steps 2 --warmup 1 > /tmp/d.json 2>/dev/null
  python -c "import json; d=json.load(open('/tmp/d.json')); print('stream event n=$n', '%.2f ms' % d['roofline']['kernel_ms'])"
done
