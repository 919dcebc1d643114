mkdir -p gpurun_out
for w in 17 15,17 3,17; do
timeout -s KILL 600 python bench.py --no-cpu-baseline --no-e2e --widths $w > gpurun_out/bench_w.json 2>/dev/null
python -c "
import json; d=json.load(open('gpurun_out/bench_w.json'))
print('$w', ' '.join('%s:%s %.0f/%.0f'%(k,v['variant'],v['tuned_us'],v['us']) for k,v in d['per_width'].items()), d['clocks']['reasons'], d['clocks'].get('power_w_max'))"
done
