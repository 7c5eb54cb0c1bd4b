# device-side bounds checks (NT_CHECKS variant) under the GPU parity suite and the
# sanitizer driver's paths -- compute-sanitizer is closed on this pool
OUT=gpurun_out/r02_chk; mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()"
bash scripts/dev/build_variants.sh "chk:-DNT_CHECKS=1" > $OUT/build.log 2>&1
NT_LIB_VARIANT=chk timeout 1500 python -m pytest tests -m gpu -q -p no:cacheprovider --ignore=tests/test_gpu_fullscale.py > $OUT/pytest_chk.log 2>&1
echo "PYTEST(checks) $(tail -1 $OUT/pytest_chk.log)"; grep -E "^FAILED|assert" $OUT/pytest_chk.log | head -5
NT_LIB_VARIANT=chk timeout 900 python scripts/sanitize_run.py > $OUT/paths_chk.log 2>&1; echo "PATHS rc=$? $(tail -1 $OUT/paths_chk.log)"
NT_LIB_VARIANT=chk timeout 900 python -m pytest tests/test_gpu_fullscale.py -m gpu -q -p no:cacheprovider -k "csp and history and default" > $OUT/fullscale_chk.log 2>&1
echo "FULLSCALE(checks) $(tail -1 $OUT/fullscale_chk.log)"
