#!/bin/bash
# round-end evidence (run under gpurun): GPU tests, smoke, every config through bench.py,
# the reference arm, the 2-rank gloo run on one GPU, ncu launch list + same-slide captures
OUT=gpurun_out/final2
mkdir -p $OUT
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
timeout 2400 python -m pytest tests -m gpu -q --timeout 900 > $OUT/pytest_gpu.log 2>&1; echo pytest rc=$?; tail -3 $OUT/pytest_gpu.log
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > $OUT/smoke.log 2>&1; echo smoke rc=$?; tail -1 $OUT/smoke.log
OUT=$OUT bash tools/configs_run.sh
timeout 900 python bench.py --impl reference --steps 3 --warmup 3 > $OUT/bench_reference.json 2> $OUT/bench_reference.err; echo reference rc=$?
timeout 900 python bench.py --gpus 2 --backend gloo --workload ms-lj --sources 64 --steps 10 --warmup 3 --no-cpu-baseline > $OUT/bench_gloo2.json 2> $OUT/bench_gloo2.err; echo gloo2 rc=$?
OUT=$OUT bash tools/profile_run.sh
