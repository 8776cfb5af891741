# SURVEY 8(f) NEXT-1 / NEXT-2 on the LJ shape (CFGFILE for tools/bench_configs.sh)
# NEXT-1: Table 3 variants (Fig. 4 ablation) on B200
for m in opt eager dupdetect vanilla scan async; do
  run abl_$m --mode $m --steps 20 --warmup 3 --no-cpu-baseline --no-e2e
done
# NEXT-2: eps sweep (Fig. 6), source at the default top-1K band
for e in 1e-4 1e-5 1e-6 1e-7 1e-8 1e-9 1e-10; do
  run eps_$e --eps $e --steps 20 --warmup 3 --no-cpu-baseline --no-e2e
done
# NEXT-2: source-degree sweep (Fig. 7): top-10 / 1K / 1M
for b in 10 1000 1000000; do
  run band_$b --band $b --steps 20 --warmup 3 --no-cpu-baseline --no-e2e
done
