# multi-source per-GPU efficiency curve (SHARED mode): S sources on one GPU = the per-rank load of
# the 256-source config at 256/S GPUs (CFGFILE for tools/bench_configs.sh)
run ms32_shared --sources 32 --steps 5 --warmup 3 --no-cpu-baseline --no-e2e --mode shared
run ms64_shared --sources 64 --steps 5 --warmup 3 --no-cpu-baseline --no-e2e --mode shared
run ms128_shared --sources 128 --steps 3 --warmup 3 --no-cpu-baseline --no-e2e --mode shared
run ms256_shared --sources 256 --steps 3 --warmup 3 --no-cpu-baseline --no-e2e --mode shared
run ms32_opt --sources 32 --steps 5 --warmup 3 --no-cpu-baseline --no-e2e --mode opt
