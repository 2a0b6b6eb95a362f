"""Write profiles/ncu_traffic.json: DRAM bytes (read + write) per launch of the probe
kernels from one `ncu --set full` capture of `bench.py` (keys config/op/b<log2>/s<bytes>)."""
import csv, json, subprocess, sys, os
rep, config, blog2, sbytes, out = sys.argv[1], sys.argv[2], sys.argv[3], sys.argv[4], sys.argv[5]
txt = subprocess.run(['ncu', '-i', rep, '--page', 'raw', '--csv'], capture_output=True, text=True).stdout
r = list(csv.reader(txt.splitlines()))
hdr, units, rows = r[0], r[1], r[2:]
scale = {'byte': 1, 'Kbyte': 1e3, 'Mbyte': 1e6, 'Gbyte': 1e9, 'Tbyte': 1e12}
ops = {'0': 'insert', '1': 'delete', '2': 'query'}
data = json.load(open(out)) if os.path.exists(out) else {}
for row in rows:
    name = row[hdr.index('Kernel Name')]
    if 'k_edges' not in name:
        continue
    op = ops[name.split('<')[1].split('>')[0].split(',')[2].strip()]  # <G, S, OP, A>
    b = 0.0
    for m in ('dram__bytes_read.sum', 'dram__bytes_write.sum'):
        i = hdr.index(m)
        b += float(row[i].replace(',', '')) * scale[units[i]]
    t = float(row[hdr.index('gpu__time_duration.sum')].replace(',', ''))
    data[f'{config}/{op}/b{blog2}/s{sbytes}'] = {
        'dram_bytes_per_launch': b, 'ncu_duration': t,
        'ncu_duration_unit': units[hdr.index('gpu__time_duration.sum')], 'source': os.path.basename(rep)}
json.dump(data, open(out, 'w'), indent=1, sort_keys=True)
print(json.dumps(data, indent=1))
