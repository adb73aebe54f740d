# Table 4 replay: parity, sanitizer, timing at 512^3, ncu counters at 256^3
mkdir -p gpurun_out/abl
timeout 900 python -m pytest tests/test_ablation.py -m gpu -q -p no:cacheprovider -x > gpurun_out/abl/pytest.txt 2>&1; echo "rc=$?" >> gpurun_out/abl/pytest.txt
tail -5 gpurun_out/abl/pytest.txt
for tool in racecheck synccheck memcheck; do
  timeout 600 compute-sanitizer --tool $tool python tools/sanitize_cases.py t4a t4b t4c t4d t4e t4f > gpurun_out/abl/san_$tool.txt 2>&1
  tail -2 gpurun_out/abl/san_$tool.txt
done
timeout 900 python tools/ablation.py time --shape 512,512,512 --T 48 > gpurun_out/abl/times.jsonl 2> gpurun_out/abl/times.err
cat gpurun_out/abl/times.jsonl | cut -c1-200
M=gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum,lts__t_bytes.sum,lts__t_sectors_srcunit_tex_op_read.sum,smsp__sass_thread_inst_executed_op_global_ld.sum,smsp__inst_executed_op_global_ld.sum,smsp__inst_executed_op_shared_ld.sum,l1tex__data_pipe_lsu_wavefronts_mem_shared_op_ld.sum,smsp__sass_average_data_bytes_per_sector_mem_global_op_ld.pct
for c in a b c d e f generic fast3d auto; do
  timeout 900 ncu --metrics $M --clock-control none -k regex:"ablation|hex3d|generic|fast3d" --csv --log-file gpurun_out/abl/abl_$c.csv python tools/ablation.py one $c --shape 256,256,256 --T 12 > /dev/null 2>&1
  echo "$c: $(grep -c ablation\\\|hex3d\\\|generic gpurun_out/abl/abl_$c.csv) rows"
done
python tools/ablation.py table gpurun_out/abl gpurun_out/abl/times.jsonl --shape 256,256,256 --T 12 > gpurun_out/abl/table.md
cat gpurun_out/abl/table.md
