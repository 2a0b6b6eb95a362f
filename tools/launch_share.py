"""Summarise an ncu --metrics gpu__time_duration.sum launch list (CSV): per kernel
name, launches, total and mean device time, and share of all library-kernel time."""
import csv, sys, collections
path = sys.argv[1]
rows = []
with open(path) as f:
    lines = [l for l in f if l.startswith('"')]
r = list(csv.reader(lines))
hdr = r[0]
ki, mi, vi, ui = hdr.index('Kernel Name'), hdr.index('Metric Name'), hdr.index('Metric Value'), hdr.index('Metric Unit')
agg = collections.OrderedDict()
for row in r[1:]:
    if row[mi] != 'gpu__time_duration.sum':
        continue
    name = row[ki].split('(')[0]
    v = float(row[vi].replace(',', ''))
    unit = row[ui]
    scale = {'nsecond': 1e-6, 'ns': 1e-6, 'usecond': 1e-3, 'us': 1e-3, 'msecond': 1.0, 'ms': 1.0}
    v = v * scale.get(unit, 1.0)  # -> ms
    a = agg.setdefault(name, [0, 0.0])
    a[0] += 1
    a[1] += v
tot = sum(a[1] for a in agg.values())
lib = {k: v for k, v in agg.items() if 'dg::' in k or k.startswith('void dg') or 'k_' in k}
ltot = sum(a[1] for a in lib.values())
print(f'{"kernel":70s} {"launches":>8s} {"total ms":>10s} {"mean ms":>9s} {"share(all)":>10s} {"share(lib)":>10s}')
for k, (n, t) in sorted(agg.items(), key=lambda x: -x[1][1]):
    sl = f'{t / ltot:10.3f}' if k in lib else f'{"-":>10s}'
    print(f'{k[:70]:70s} {n:8d} {t:10.3f} {t / n:9.4f} {t / tot:10.3f} {sl}')
print(f'total {tot:.3f} ms, library kernels {ltot:.3f} ms')
