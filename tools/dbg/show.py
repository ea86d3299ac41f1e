import json
d=json.load(open('gpurun_out/bench_count.json')); print('bench ms', d['ms_per_step'], {k: round(v['ms'],3) for k,v in d['roofline']['classes'].items()})
d=json.load(open('gpurun_out/rounds_count.json'))
for b in d['buckets']:
    r=b['rounds']; nr=r[1]-r[0]; s=b['stat_sums']
    print(r, 'round %.1f'%(s[4]/nr/1e3), 'tgt %.1f'%(s[6]/nr/1e3), 'units_max %.1f'%(s[7]/nr/1e3), 'units_min %.1f'%(s[9]/nr/1e3), 'flushstart %.1f'%(s[5]/nr/1e3), 'flushend %.1f'%(s[8]/nr/1e3), 'unitcyc %.0f'%(s[10]/nr), 'entries %d'%(s[2]/nr), 'fresh mean %.2f max %.2f maxnf %.0f'%(s[11]/nr/148/1e3, s[12]/nr/1e3, s[13]/nr))
