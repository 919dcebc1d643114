mkdir -p gpurun_out
for r in 1 2 3; do
timeout -s KILL 900 python bench.py --no-cpu-baseline > gpurun_out/bench_pc_$r.json 2>/dev/null
python tools/bench_summary.py gpurun_out/bench_pc_$r.json
python -c "
import json; d=json.load(open('gpurun_out/bench_pc_$r.json'))
print(' '.join('%s:%.0f/%.0f'%(k,v['tuned_us'],v['us']) for k,v in d['per_width'].items()), d['clocks'])"
done
