#!/bin/bash
# under gpurun: build, full GPU tests, default bench, 2-rank gloo bench on one GPU, A/B variants
mkdir -p gpurun_out/chk
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
timeout 1500 python -m pytest tests -m gpu -q --timeout 600 -x > gpurun_out/chk/pytest_gpu.log 2>&1; echo pytest rc=$?; tail -5 gpurun_out/chk/pytest_gpu.log
timeout 900 python bench.py > gpurun_out/chk/bench.json 2> gpurun_out/chk/bench.err; echo bench rc=$?; tail -c 300 gpurun_out/chk/bench.err
timeout 900 python bench.py --gpus 2 --backend gloo --workload ms-lj --sources 64 --steps 10 --warmup 3 --no-cpu-baseline > gpurun_out/chk/bench_gloo2.json 2> gpurun_out/chk/bench_gloo2.err; echo gloo2 rc=$?; tail -c 600 gpurun_out/chk/bench_gloo2.err
[ -d build/variants ] && REPS=2 PARITY_K="test_tiny_config_all_modes_track_oracle and opt" bash tools/dev/gpu_ab.sh
