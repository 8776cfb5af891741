# SHARED tile / queue-slice variants with external ids (build/variants/libppr_*.so)
mkdir -p gpurun_out/msvar2
for rep in 1 2; do
for lib in build/variants/libppr_*.so; do
  name=$(basename $lib .so)
  for cfg in "s0of8 --shard 0/8" "s256"; do
    set -- $cfg; tag=$1; shift
    PPR_LIB=$PWD/$lib timeout 600 python bench.py --sources 256 --mode shared --steps 5 --warmup 3 --no-cpu-baseline --no-e2e "$@" > gpurun_out/msvar2/${name}_${tag}_$rep.json 2> gpurun_out/msvar2/${name}_${tag}_$rep.err
    python -c "import json;d=json.load(open('gpurun_out/msvar2/${name}_${tag}_$rep.json'));x=d['detail'];print('$name $tag $rep', 'step %.3f push %.3f' % (d['ms_per_step'], x['ms_push']))" 2>/dev/null || { echo "$name $tag failed"; tail -2 gpurun_out/msvar2/${name}_${tag}_$rep.err; }
  done
done
done
