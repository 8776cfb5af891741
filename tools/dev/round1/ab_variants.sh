#!/bin/bash
# dev helper: short LJ bench for each build/variants/libppr_*.so (run under gpurun)
mkdir -p gpurun_out
for lib in build/variants/libppr_*.so; do
  name=$(basename $lib .so)
  PPR_LIB=$PWD/$lib timeout 300 python bench.py --steps 20 --warmup 3 --no-cpu-baseline --no-e2e ${BENCH_ARGS} > gpurun_out/ab_$name.json 2> gpurun_out/ab_$name.err
  python -c "import json,sys;d=json.load(open('gpurun_out/ab_$name.json'));x=d['detail'];print('$name', 'step %.3f push %.3f edges %.3g iters %.1f' % (d['ms_per_step'], x['ms_push'], x['pushed_edges_per_step'], x['iters_per_step']))" 2>/dev/null || echo "$name failed"
done
