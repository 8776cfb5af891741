#!/bin/bash
# A/B of build/variants + per-round trace of each (run under gpurun)
mkdir -p gpurun_out/abt
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
REPS=${REPS:-2} PARITY_K="${PARITY_K:-test_tiny_config_all_modes_track_oracle and opt or test_opt_schedules}" BENCH_ARGS="--no-multi-source $BENCH_ARGS" bash tools/dev/gpu_ab.sh
for lib in build/variants/libppr_*.so; do
  name=$(basename $lib .so)
  PPR_TRACE=1 PPR_LIB=$PWD/$lib timeout 300 python bench.py --steps 2 --warmup 3 --no-cpu-baseline --no-e2e --no-multi-source $BENCH_ARGS > /dev/null 2> gpurun_out/abt/trace_$name.err
  echo "$name tails: $(grep 'PPR_TRACE apply' gpurun_out/abt/trace_$name.err | tail -1 | tr ']' '\n' | grep -E ' 0 [0-9.]+us' | tr '\n' ' ')"
done
