# session-5 final check: full GPU suite, smoke, default bench, the multi-source pair under the final rule
timeout 1200 python -m pytest tests -m gpu -q --timeout 300 > gpurun_out/pytest_gpu.log 2>&1; echo pytest rc=$?; tail -2 gpurun_out/pytest_gpu.log
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/smoke.log 2>&1; echo smoke rc=$?; tail -1 gpurun_out/smoke.log
run lj --steps 100 --warmup 5
run ms256 --sources 256 --steps 5 --warmup 3 --no-cpu-baseline --no-e2e
run ms256_s3of8 --sources 256 --shard 3/8 --steps 5 --warmup 3 --no-cpu-baseline --no-e2e
