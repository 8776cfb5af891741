# multi-source handles keep external ids by default: refresh of the multi-source configs
timeout 900 python -m pytest tests -m gpu -q --timeout 300 -k "multi or shared or sortagg or ms" > gpurun_out/pytest_gpu.log 2>&1; echo pytest rc=$?; tail -2 gpurun_out/pytest_gpu.log
run ms256 --sources 256 --steps 5 --warmup 3 --no-cpu-baseline --no-e2e --mode shared
run ms16 --sources 16 --steps 5 --warmup 3 --no-cpu-baseline --no-e2e --mode shared
run ms4_opt --sources 4 --steps 5 --warmup 3 --no-cpu-baseline --no-e2e --mode opt
run ms4_opt_relabel --sources 4 --steps 5 --warmup 3 --no-cpu-baseline --no-e2e --mode opt --relabel 1
for r in 0 1 2 3 4 5 6 7; do run ms256_s${r}of8 --sources 256 --shard $r/8 --steps 5 --warmup 3 --no-cpu-baseline --no-e2e --mode shared; done
for r in 0 1 2 3; do run ms256_s${r}of4 --sources 256 --shard $r/4 --steps 5 --warmup 3 --no-cpu-baseline --no-e2e --mode shared; done
for r in 0 1; do run ms256_s${r}of2 --sources 256 --shard $r/2 --steps 5 --warmup 3 --no-cpu-baseline --no-e2e --mode shared; done
